#!/bin/bash
# Medium window width (LMOSEM_ZMWIN, voxels; 0 = the coarse slab width, 188 at C4) at C4.
O=gpurun_out/zmwin
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1 || { echo BUILD FAILED; exit 1; }
LMOSEM_ZMWIN=${ZMW_TEST:-230} timeout 600 python -m pytest tests/test_zlist_gpu.py -q -p no:cacheprovider -x 2>&1 | tail -1
for rep in 1 2; do for w in ${ZMW_LIST:-0 160 210 230 260}; do
  LMOSEM_ZMED=${ZMW_MED:-6} LMOSEM_ZMWIN=$w timeout 400 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_${w}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${w}_r$rep.json'));print('C4 zmwin=$w', round(d['ms_per_step'],3))" 2>&1 | tail -1
done; done
