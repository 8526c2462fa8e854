#!/bin/bash
# z-slab pass A with texture gathers (variants/liblmosem_atex.so, LMK_PASSA_TEX=1) vs LSU gathers (new).
O=gpurun_out/passa_tex
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1 || { echo BUILD FAILED; exit 1; }
timeout 900 python -m pytest tests/test_zlist_gpu.py tests/test_loopback_gpu.py tests/test_parity_gpu.py -q -p no:cacheprovider -x -k "listed or zslab or c4 or sensitivity" > $O/pytest.txt 2>&1; tail -1 $O/pytest.txt
for rep in 1 2 3; do for v in ${LW_VARIANTS:-atex new}; do
  if [ $v = new ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L timeout 400 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_${v}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${v}_r$rep.json'));s=d['per_rank_share'];print('C4 $v', round(d['ms_per_step'],3), round(d['phase_ms_per_step']['project'],3), [round(s[k]['loop_ms_per_subset'],3) for k in ('2','4','8')])" 2>&1 | tail -1
done; done
