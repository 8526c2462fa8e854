#!/bin/bash
# Round-2 evidence on one B200 (run through gpurun): the GPU suite with per-test parity
# errors, bench lines (C2 default, C5, C4, the oracle arm, torchrun N=1), the ncu launch
# list of the bench command, smoke(), ncu --set full of the C2/C5 projection and the update,
# C4 z-slab DRAM per subset cold (ncu default cache control) and warm (--cache-control none),
# the combine forms on a 1-rank communicator. Output: gpurun_out/ev2/ (summaries copied to
# profiles/r02_final_* by hand).
O=gpurun_out/ev2
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1
(echo "# pytest -m gpu -v -s (one B200): per-test parity errors vs the float64 oracle"; timeout 1500 python -m pytest tests -m gpu -v -s -p no:cacheprovider 2>&1 | grep -E "parity|watchdog|PASSED|FAILED|passed|failed|Error") > $O/parity.txt
python bench.py > $O/bench_C2.json 2> $O/bench_C2.err
python bench.py --config C5 > $O/bench_C5.json 2> /dev/null
python bench.py --config C4 --steps 20 > $O/bench_C4.json 2> /dev/null
python bench.py --impl reference > $O/bench_reference.json 2> /dev/null
python -m torch.distributed.run --nnodes 1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29511 \
    bench.py --gpus 1 > $O/bench_torchrun_n1.json 2> /dev/null
python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" > $O/smoke.txt 2>&1
python tools/combine_1rank.py > $O/combine_1rank.txt 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $O/launches.csv \
    python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
python tools/launch_shares.py $O/launches.csv > $O/launches_summary.txt 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_project -s 3 -c 1 -o $O/k_project_C2 \
    python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_project -s 3 -c 1 -o $O/k_project_C5 \
    python bench.py --config C5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
ncu --set full --clock-control none -k regex:k_update -s 3 -c 1 -o $O/k_update_C2 \
    python bench.py --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
for cc in all none; do
  ncu --cache-control $cc --clock-control none --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum,lts__t_sectors_srcunit_tex_op_read.sum,lts__t_sectors_srcunit_tex_op_red.sum \
      -k regex:k_project -s 18 -c 6 --csv --log-file $O/c4_dram_cache_$cc.csv \
      python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
done
for r in k_project_C2 k_project_C5 k_update_C2; do python tools/ncu_summary.py $O/$r.ncu-rep > $O/${r}_summary.txt 2>&1; done
ls -la $O
