O=gpurun_out/c5_ncu
mkdir -p $O
M=gpu__time_duration.sum,launch__grid_size,launch__block_size,launch__shared_mem_per_block_dynamic,launch__registers_per_thread,launch__occupancy_limit_shared_mem,sm__inst_executed.sum,lts__t_sectors_srcunit_tex_op_red.sum,lts__t_sectors_srcunit_tex_op_read.sum
for v in prev new; do
  if [ $v = new ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L ncu --clock-control none --metrics $M -k regex:k_project -s 20 -c 3 --csv --log-file $O/$v.csv python bench.py --config C5 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
done
