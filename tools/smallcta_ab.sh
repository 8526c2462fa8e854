O=gpurun_out/smallcta
mkdir -p $O
LMOSEM_SMALL_CTA_N=2000000 timeout 600 python -m pytest tests/test_parity_gpu.py -x -q -p no:cacheprovider -k "c1_ or one_subset_paper or golden or degenerate or odd_extents" 2>&1 | tail -1
for rep in 1 2; do
 for t in 0 600000 2000000; do
  for c in C2 C5; do
   LMOSEM_SMALL_CTA_N=$t python bench.py --config $c --no-cpu-baseline --no-e2e --steps 100 > $O/b_${c}_t${t}_r$rep.json 2>/dev/null
   python -c "import json;d=json.load(open('$O/b_${c}_t${t}_r$rep.json'));s=d['per_rank_share'];print('$c t=$t', round(d['ms_per_step'],4), [round(s[k]['project_ms'],4) for k in ('2','4','8')], round(s['8']['loop_ms_per_subset'],4))"
  done
 done
done
