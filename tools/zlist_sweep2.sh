#!/bin/bash
# Coarse slab count and window width around the kept point (merged windows, stride W/4).
O=gpurun_out/zlist_sweep2
mkdir -p $O
for rep in 1 2; do
for v in 3_0 4_92 4_0 3_88 3_96; do set -- ${v//_/ }
  LMOSEM_ZWIN=$2 timeout 300 python bench.py --config C4 --steps 10 --slabs $1 --no-cpu-baseline --no-e2e > $O/b_$1_$2_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_$1_$2_r$rep.json'));print('C4 slabs=$1 zwin=$2', round(d['ms_per_step'],3))" 2>&1 | tail -1
done; done
