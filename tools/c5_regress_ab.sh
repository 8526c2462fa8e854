#!/bin/bash
# C2/C5 with the previous library (variants/liblmosem_prev.so) vs the current one, alternating.
O=gpurun_out/c5_ab
mkdir -p $O
for rep in 1 2 3; do
 for v in prev new; do
  if [ $v = new ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C5 C2; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));print('$c $v', round(d['ms_per_step'],4))" 2>&1 | tail -1
  done
 done
done
