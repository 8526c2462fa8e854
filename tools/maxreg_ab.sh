#!/bin/bash
# (round 2, no difference: C2 0.9361 vs 0.9363, C5 1.7450 vs 1.7451, shares equal) A/B: the library built with -maxrregcount=72 (caps MODE 5 at 72 registers) vs default.
O=gpurun_out/rr; mkdir -p $O
for rep in 1 2; do for v in default rr72; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')])"
  done
done; done
