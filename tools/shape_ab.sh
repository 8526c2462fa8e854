#!/bin/bash
# A/B of the fused pass's CTA shape (threads x resident CTAs per SM; variants/liblmosem_t<T>b<B>.so
# built with LMK_CTA_THREADS / LMK_MIN_BLOCKS) at C2 and C5: full subset and the per-rank shares.
O=gpurun_out/shape_ab
mkdir -p $O
for rep in 1 2; do
 for v in default t224b4 t128b7 t96b9 t64b14 t160b5; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')], round(s['8']['loop_ms_per_subset'],4))" 2>&1 | tail -1
  done
 done
done
