#!/bin/bash
# (round 2, rejected; switch removed) A/B: LMK_DEFER_ACC=1 (a round's gathers accumulated one round later) vs default.
O=gpurun_out/defer
mkdir -p $O
for rep in 1 2 3; do for v in default defer; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 200 > $O/b_${c}_${v}_$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_$rep.json'));p=d['phase_ms_per_step'];print('$c $v', round(d['ms_per_step'],4), round(p['project'],4), round(p['update'],4))"
  done
done; done
