#!/bin/bash
# (round 2, rejected and removed) Experiment: the LOR setup of small launches in its own kernel (k_lor_setup + MODE 7,
# LMOSEM_PRESETUP=1) vs the claim-time setup (MODE 5).
O=gpurun_out/presetup_ab
mkdir -p $O
LMOSEM_PRESETUP=1 timeout 900 python -m pytest tests/test_parity_gpu.py -x -q -p no:cacheprovider -k "c1_ or golden or degenerate or odd_extents or axis_parallel or faces" 2>&1 | tail -1
for rep in 1 2; do
 for v in 0 1; do
  for c in C2 C5; do
   LMOSEM_PRESETUP=$v python bench.py --config $c --no-cpu-baseline --no-e2e --steps 50 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c presetup=$v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')], round(s['8']['loop_ms_per_subset'],4))" 2>&1 | tail -1
  done
 done
done
