#!/bin/bash
# Listed vs unlisted z-slab form at a rank's share of a C4 subset (P = 1, 2, 4, 8).
O=gpurun_out/zlist_share
mkdir -p $O
for rep in 1 2; do for z in 0 2; do
  LMOSEM_ZLIST=$z timeout 400 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_z${z}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_z${z}_r$rep.json'));s=d['per_rank_share'];print('C4 zlist=$z full', round(d['ms_per_step'],3), 'shares', [(k, round(s[k]['project_ms'],3), round(s[k]['loop_ms_per_subset'],3)) for k in ('2','4','8')])"
done; done
