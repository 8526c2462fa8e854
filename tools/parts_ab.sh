#!/bin/bash
# A/B of claim partitions (LMOSEM_CLAIM_PARTS: the events of a launch in P contiguous ranges,
# one claim counter each) against the single-counter kernel (variants/liblmosem_prev.so).
O=gpurun_out/parts_ab
mkdir -p $O
LMOSEM_CLAIM_PARTS=8 timeout 900 python -m pytest tests/test_parity_gpu.py tests/test_loopback_gpu.py -x -q -p no:cacheprovider -k "c1_ or one_subset_paper or zslab or odd_extents or golden or loopback_c1 or shapes or degenerate" 2>&1 | tail -1
for rep in 1 2; do
 for v in prev p1 p2 p4 p8 p16; do
  case $v in prev) L=variants/liblmosem_prev.so; P=1;; p*) L=""; P=${v#p};; esac
  for c in C2 C5; do
   LMOSEM_LIB=$L LMOSEM_CLAIM_PARTS=$P python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')], round(s['8']['loop_ms_per_subset'],4))" 2>&1 | tail -1
  done
 done
done
