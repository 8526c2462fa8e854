#!/bin/bash
# (round 2; the mixed kernel was rejected and removed, see profiles/r02_mix_ab) A/B of the mixed z-slab schedule (k_project_mix: pass A of chunk r with pass B of chunk r-1
# in one launch) at C4: parity first, then bench lines over chunks x slabs x CTA shape.
O=gpurun_out/mix_ab
mkdir -p $O
LMOSEM_MIX_CHUNKS=4 LMOSEM_MIX_SLABS=4 timeout 900 python -m pytest tests/test_parity_gpu.py -x -q -p no:cacheprovider \
    -k "zslab or c4_full_subset or c4_full_size or odd_extents" > $O/parity_mix.txt 2>&1
tail -1 $O/parity_mix.txt
run() {  # name, env...
  local name=$1; shift
  env "$@" python bench.py --config C4 --steps 10 --warmup 3 --no-cpu-baseline --no-e2e > $O/b_$name.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_$name.json'));print('$name', round(d['ms_per_step'],3), round(d['phase_ms_per_step']['project'],3), d['clocks']['reasons'])"
}
for rep in 1 2; do
  run base_r$rep LMOSEM_MIX_CHUNKS=0
  run m2k3_r$rep LMOSEM_MIX_CHUNKS=2
  run m4k3_r$rep LMOSEM_MIX_CHUNKS=4
  run m4k4_r$rep LMOSEM_MIX_CHUNKS=4 LMOSEM_MIX_SLABS=4
  run m4k5_r$rep LMOSEM_MIX_CHUNKS=4 LMOSEM_MIX_SLABS=5
  run m8k4_r$rep LMOSEM_MIX_CHUNKS=8 LMOSEM_MIX_SLABS=4
  run m4k4_cta5_r$rep LMOSEM_MIX_CHUNKS=4 LMOSEM_MIX_SLABS=4 LMOSEM_LIB=variants/liblmosem_mix5.so
done
