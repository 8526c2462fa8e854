#!/bin/bash
# Round-end evidence on one B200 (run through gpurun): parity errors, bench lines
# (C2 default, C5, C4, the oracle arm, torchrun N=1), the ncu launch list of the bench
# command and smoke(). Output: gpurun_out/ev/ (copied to profiles/ by hand).
O=gpurun_out/ev
mkdir -p $O
(echo "# pytest -m gpu -v -s (one B200): per-test parity errors vs the float64 oracle"; python -m pytest tests -m gpu -v -s -p no:cacheprovider 2>&1 | grep -E "parity|PASSED|FAILED|passed|failed|Error") > $O/parity.txt
python bench.py > $O/bench_C2.json 2> $O/bench_C2.err
python bench.py --config C5 > $O/bench_C5.json 2> /dev/null
python bench.py --config C4 --steps 20 > $O/bench_C4.json 2> /dev/null
python bench.py --impl reference > $O/bench_reference.json 2> /dev/null
python -m torch.distributed.run --nnodes 1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29511 \
    bench.py --gpus 1 > $O/bench_torchrun_n1.json 2> /dev/null
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $O/launches.csv \
    python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" > $O/smoke.txt 2>&1
# ncu --set full of the C2 projection (traffic for bench.py), C5, and the update kernel
ncu --set full --clock-control none --import-source on -k regex:k_project -s 3 -c 1 -o $O/k_project_C2 \
    python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_project -s 3 -c 1 -o $O/k_project_C5 \
    python bench.py --config C5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
ncu --set full --clock-control none -k regex:k_update -s 3 -c 1 -o $O/k_update_C2 \
    python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
