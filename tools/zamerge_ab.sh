#!/bin/bash
# Pass A of all coarse slabs in one launch (LMOSEM_ZAMERGE=1) vs one per slab (0).
O=gpurun_out/zamerge
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1 || { echo BUILD FAILED; exit 1; }
LMOSEM_ZAMERGE=1 timeout 600 python -m pytest tests/test_zlist_gpu.py tests/test_loopback_gpu.py -q -p no:cacheprovider -x -k listed > $O/pytest.txt 2>&1; tail -1 $O/pytest.txt
for rep in 1 2 3; do for v in 0 1; do
  LMOSEM_ZAMERGE=$v timeout 400 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_${v}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${v}_r$rep.json'));s=d['per_rank_share'];print('C4 zamerge=$v', round(d['ms_per_step'],3), [round(s[k]['loop_ms_per_subset'],3) for k in ('2','4','8')])" 2>&1 | tail -1
done; done
