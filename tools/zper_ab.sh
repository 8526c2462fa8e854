#!/bin/bash
# k_zclass events per thread (LMK_ZPER 4 / 8 / 16): C4 ms per subset and the classifier's time.
O=gpurun_out/zper_ab
mkdir -p $O
for rep in 1 2; do for v in zper1 zper2 zper4 new; do
  if [ $v = new ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L timeout 300 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_${v}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${v}_r$rep.json'));print('C4 $v', round(d['ms_per_step'],3))" 2>&1 | tail -1
done; done
for v in zper1 zper2 zper4 new; do
  if [ $v = new ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L ncu --clock-control none --metrics gpu__time_duration.sum,sm__inst_executed.sum -k regex:k_zclass -s 3 -c 2 --csv --log-file $O/ncu_$v.csv python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
  echo $v; python tools/ncu_launch_table.py $O/ncu_$v.csv
done
