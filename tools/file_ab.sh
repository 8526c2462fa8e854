mkdir -p gpurun_out
for v in read1 read2 read3 read4 read6 read4 read2; do
  LMOSEM_LIB=variants/liblmosem_$v.so python bench.py --steps 20 --warmup 3 --no-cpu-baseline --e2e-file 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$v', d['e2e']['value'], d['e2e']['file']['value'])" >> gpurun_out/file_ab.log
done
nproc >> gpurun_out/file_ab.log
