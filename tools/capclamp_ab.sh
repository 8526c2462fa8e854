#!/bin/bash
# Timing-only A/B (round 2): the fused pass's path buffer clamped below the Σe + 4 bound
# (variants/liblmosem_cap<N>.so built with -DLMOSEM_CAP_CLAMP=N -DLMK_CAP_GUARD=1: a clamp in
# launch_cap and a per-LOR piece bound that drops LORs with more pieces, both test-only patches
# kept in profiles/r02_capclamp_ab/summary.txt, never used for parity): does a smaller shared-
# memory footprint (the 132 KB carveout, 124 KB of L1) pay at C2?
O=gpurun_out/capclamp_ab
mkdir -p $O
for rep in 1 2 3; do
 for v in default cap520 cap488 cap456; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L python bench.py --config C2 --no-cpu-baseline --no-e2e --steps 100 > $O/b_C2_${v}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_C2_${v}_r$rep.json'));s=d['per_rank_share'];print('C2 $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')])" 2>&1 | tail -1
 done
done
