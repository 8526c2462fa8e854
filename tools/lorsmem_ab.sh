#!/bin/bash
# Round 2: LOR records in shared memory (lor_store / lor_load) instead of 16 shuffles per LOR
# vs the previous tree (variants/liblmosem_prev.so).
O=gpurun_out/lorsmem_ab3
mkdir -p $O
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -1
for rep in 1 2 3; do
 for v in prev new; do
  if [ $v = new ]; then L=""; else L=variants/liblmosem_$v.so; fi
  for c in C2 C5; do
   LMOSEM_LIB=$L python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${v}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_${v}_r$rep.json'));s=d['per_rank_share'];print('$c $v', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')])" 2>&1 | tail -1
  done
  LMOSEM_LIB=$L python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_C4_${v}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_C4_${v}_r$rep.json'));print('C4 $v', round(d['ms_per_step'],3))" 2>&1 | tail -1
 done
done
