O=gpurun_out/zmed2
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for rep in 1 2; do for z in 4 6 8 10; do
  LMOSEM_ZMED=$z timeout 400 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_${z}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${z}_r$rep.json'));print('C4 zmed=$z', round(d['ms_per_step'],3), d['clocks']['reasons'])" 2>&1 | tail -1
done; done
