#!/bin/bash
# Long fuzz of the final tree (listed z-slab form included: slabs 0-4 at random per case).
O=gpurun_out/fuzz_r02b
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1 || { echo BUILD FAILED; exit 1; }
LMOSEM_FUZZ_CASES=2400 LMOSEM_FUZZ_SEED0=30000 timeout 1800 python -m pytest tests/test_fuzz_gpu.py -q -p no:cacheprovider -k "matches_oracle or loopback_world or reconstruct_paths" > $O/fuzz.txt 2>&1
tail -3 $O/fuzz.txt
