#!/bin/bash
# (round 2, variants since removed) A/B of the update kernel grid (LMOSEM_UPDATE_GRID) at C2.
O=gpurun_out/ug; mkdir -p $O
for rep in 1 2 3; do for v in default ug1 ug2; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L python bench.py --no-cpu-baseline --no-e2e --steps 200 > $O/b_${v}_$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${v}_$rep.json'));print('$v', round(d['ms_per_step'],4), round(d['phase_ms_per_step']['update'],4))"
done; done
