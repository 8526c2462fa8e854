#!/bin/bash
# A/B: path buffers sized by min(3 max e, sum e + 4) (default) vs 3 max e (variants/liblmosem_cap3.so),
# for the one-warp-per-claim kernel and (round 2, since removed) the warp-specialised one (LMOSEM_WS=1).
O=gpurun_out/cap_ab
mkdir -p $O
timeout 900 python -m pytest tests/test_parity_gpu.py -x -q -p no:cacheprovider -k "c1_ or one_subset_paper or odd_extents or golden or zslab or c4_full_subset" > $O/parity.txt 2>&1
tail -1 $O/parity.txt
for rep in 1 2; do
  for lib in default cap3; do
    if [ $lib = default ]; then L=""; else L=variants/liblmosem_cap3.so; fi
    for ws in 0 1; do
      for c in C2 C5; do
        LMOSEM_LIB=$L LMOSEM_WS=$ws python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_${lib}_ws${ws}_r$rep.json 2>/dev/null
      done
    done
    LMOSEM_LIB=$L python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_C4_${lib}_ws0_r$rep.json 2>/dev/null
  done
done
python - <<'PY'
import json, glob
for f in sorted(glob.glob("gpurun_out/cap_ab/b_*.json")):
    try:
        d = json.load(open(f))
    except Exception as e:
        print(f, "ERR", e); continue
    sh = d.get("per_rank_share") or {}
    s8 = sh.get("8", {})
    print(f.split("/")[-1], "ms/subset %.4f" % d["ms_per_step"], "proj %.4f" % d["phase_ms_per_step"]["project"],
          "1/8 proj %.4f loop %.4f" % (s8.get("project_ms", 0), s8.get("loop_ms_per_subset", 0)))
PY
