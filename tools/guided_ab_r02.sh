#!/bin/bash
# A/B of the guided-claim divisor of large launches (MODE 6) at C2 / C5 whole subsets.
O=gpurun_out/guided_r02
mkdir -p $O
for rep in 1 2; do
 for v in default gl2 gl4 gr4; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));print('$c $v', round(d['ms_per_step'],4))" 2>&1 | tail -1
  done
 done
done
