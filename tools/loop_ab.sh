#!/bin/bash
# A/B of geometry-loop variants on the peeled kernel: middle-round unroll 1 / 2 (default: the
# compiler's choice) and the two-ballot path-buffer prefix (LMK_APPEND2).
O=gpurun_out/loop_ab
mkdir -p $O
for rep in 1 2; do
 for v in default u1 u2 a2; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')])" 2>&1 | tail -1
  done
 done
done
