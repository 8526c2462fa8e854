#!/bin/bash
# (round 2, no effect; switch removed) A/B: k_update reading c with plain loads (variants/liblmosem_upc.so) vs evict-first __ldcs.
O=gpurun_out/upc
mkdir -p $O
for rep in 1 2 3; do for v in default upc; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 200 > $O/b_${c}_${v}_$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_$rep.json'));p=d['phase_ms_per_step'];print('$c $v', round(d['ms_per_step'],4), round(p['project'],4), round(p['update'],4))"
  done
done; done
