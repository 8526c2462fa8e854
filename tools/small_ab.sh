mkdir -p gpurun_out
for v in default min2 claims8 claims2 default; do
  echo -n "$v " >> gpurun_out/small_ab.log
  LMOSEM_LIB=variants/liblmosem_$v.so PYTHONPATH=. python tools/small_subsets.py 2>&1 | python -c "import json,sys; d=json.load(sys.stdin); print({k: round(v['project_ms'],4) for k,v in d.items()})" >> gpurun_out/small_ab.log
done
