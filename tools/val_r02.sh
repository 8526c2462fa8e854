O=gpurun_out/val1
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > $O/pytest_gpu.txt 2>&1
tail -3 $O/pytest_gpu.txt
python bench.py > $O/bench_C2.json 2> $O/bench_C2.err
python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/bench_C4.json 2> /dev/null
python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" > $O/smoke.txt 2>&1
tail -1 $O/smoke.txt
python -c "import json;d=json.load(open('$O/bench_C2.json'));print('C2',d['ms_per_step'],d['value']);d=json.load(open('$O/bench_C4.json'));print('C4',d['ms_per_step'])"
