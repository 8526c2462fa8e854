#!/bin/bash
# Round 2 (listed z-slab form): GPU suite, C4 traffic capture of the listed launches (updates
# profiles/r02_traffic.json C4 on the box copy; copied back by hand), ncu --set full of a
# pass-B and a fine-window launch, bench lines C2/C4/C5 + reference, smoke, launch list.
O=gpurun_out/${EV_OUT:-ev3}
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1 || { echo BUILD FAILED; tail -5 $O/build.txt; exit 1; }
(echo "# pytest -m gpu -v -s (one B200): per-test parity errors vs the float64 oracle"; timeout 1500 python -m pytest tests -m gpu -v -s -p no:cacheprovider 2>&1 | grep -E "parity|watchdog|PASSED|FAILED|passed|failed|Error") > $O/parity.txt
tail -1 $O/parity.txt
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_srcunit_tex_op_read.sum,lts__t_sectors_srcunit_tex_op_red.sum,lts__t_requests_srcunit_tex_op_read.sum,lts__t_requests_srcunit_tex_op_red.sum,l1tex__m_l1tex2xbar_req_cycles_active.avg.pct_of_peak_sustained_elapsed,sm__inst_executed.sum,smsp__issue_active.avg.pct_of_peak_sustained_active
ncu --clock-control none --metrics $M -k regex:k_project -s 27 -c 9 -o $O/c4_listed_traffic python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > $O/ncu_traffic.log 2>&1
LMOSEM_TRAFFIC_JSON=$O/r02_traffic.json cp profiles/r02_traffic.json $O/r02_traffic.json
LMOSEM_TRAFFIC_JSON=$O/r02_traffic.json python tools/update_traffic.py $O/c4_listed_traffic.ncu-rep r02_c4_listed_traffic.txt C4 9 listed > $O/update_traffic.txt 2>&1
ncu -i $O/c4_listed_traffic.ncu-rep --page raw --csv > $O/c4_listed_traffic.csv 2>/dev/null
cp $O/r02_traffic.json profiles/r02_traffic.json
ncu --set full --clock-control none --import-source on -k regex:k_project -s 35 -c 1 -o $O/k_project_C4_passB python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_project -s 32 -c 1 -o $O/k_project_C4_window python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
for r in k_project_C4_passB k_project_C4_window; do python tools/ncu_summary.py $O/$r.ncu-rep > $O/${r}_summary.txt 2>&1; done
python bench.py > $O/bench_C2.json 2> $O/bench_C2.err
python bench.py --config C5 > $O/bench_C5.json 2> /dev/null
python bench.py --config C4 --steps 20 > $O/bench_C4.json 2> /dev/null
LMOSEM_ZLIST=0 python bench.py --config C4 --steps 20 --no-cpu-baseline --no-e2e > $O/bench_C4_unlisted.json 2> /dev/null
python bench.py --impl reference > $O/bench_reference.json 2> /dev/null
python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" > $O/smoke.txt 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $O/launches.csv \
    python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
python tools/launch_shares.py $O/launches.csv > $O/launches_summary.txt 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $O/launches_C4.csv \
    python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
python tools/launch_shares.py $O/launches_C4.csv > $O/launches_C4_summary.txt 2>&1
for c in C2 C4 C5; do python -c "import json;d=json.load(open('$O/bench_$c.json'));print('$c', round(d['ms_per_step'],4), '%.4g'%d['value'], d['roofline'].get('frac'), (d.get('roofline_l2_requests') or {}).get('frac'))"; done
ls $O
