#!/bin/bash
# A/B of the CTA shape of the small-launch fused pass (MODE 5; the per-rank shares at P >= 2;
# whole subsets run MODE 6) — variants/liblmosem_s<T>b<B>.so.
O=gpurun_out/share_shape_ab
mkdir -p $O
for rep in 1 2; do
 for v in default s256b2 s192b3 s192b4 s128b6 s128b5; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 30 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')], round(s['8']['loop_ms_per_subset'],4))" 2>&1 | tail -1
  done
 done
done
