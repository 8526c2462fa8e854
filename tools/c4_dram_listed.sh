#!/bin/bash
# DRAM bytes of one C4 subset's listed launches (k_zclass + 9 k_project), ncu cache control
# all (cold: L2 flushed before each launch) vs none (warm: as the loop runs).
O=gpurun_out/c4_dram
mkdir -p $O
for cc in all none; do
  ncu --cache-control $cc --clock-control none --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum \
      -k regex:"k_project|k_zclass" -s 30 -c 10 --csv --log-file $O/c4_dram_$cc.csv \
      python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
done
