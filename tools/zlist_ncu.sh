O=gpurun_out/zlist_ncu
mkdir -p $O
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sector_hit_rate.pct,sm__warps_active.avg.pct_of_peak_sustained_active,launch__occupancy_limit_shared_mem,launch__grid_size,launch__block_size,sm__inst_executed.sum
for v in "2 2" "1 2" "2 1"; do set -- $v
LMOSEM_ZLIST=$1 LMOSEM_ZFINE=$2 ncu --clock-control none --metrics $M -k regex:"k_project|k_zclass" -s 40 -c 40 --csv --log-file $O/z$1_$2.csv python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
done
ls -la $O
