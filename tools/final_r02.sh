EV_OUT=${EV_OUT:-ev7} bash tools/evidence_r02b.sh
bash tools/fuzz_long_r02b.sh
python tools/gpu_mutants.py run "listed:" > gpurun_out/${MUT_OUT:-mutants_listed5.txt} 2>&1; grep -E "^(ok|BROKEN|killed|SURVIVED)" gpurun_out/${MUT_OUT:-mutants_listed5.txt}
