#!/bin/bash
# Round 2: listed z-slab form (k_zclass lists; LMOSEM_ZLIST 0/1/2, fine slabs per coarse slab
# LMOSEM_ZFINE, fused mode LMOSEM_ZFUSED_MODE) at C4, after the parity tests; then the
# per-launch ncu list (gpu time, DRAM, hit rate) of one subset per form.
O=gpurun_out/${ZAB_OUT:-zlist_ab}
mkdir -p $O
python -c "import __graft_entry__ as g; g.build()" > $O/build.txt 2>&1 || { echo BUILD FAILED; tail -5 $O/build.txt; exit 1; }
timeout 900 python -m pytest tests/test_zlist_gpu.py -q -p no:cacheprovider -x > $O/pytest_zlist.txt 2>&1; tail -2 $O/pytest_zlist.txt
timeout 900 python -m pytest tests/test_parity_gpu.py -q -p no:cacheprovider -x -k "zslab or c4 or sensitivity" > $O/pytest_slab.txt 2>&1; tail -2 $O/pytest_slab.txt
for rep in 1 2; do
 IFS=',' read -ra FORMS <<< "${ZAB_FORMS:-0_2_6_1,1_2_6_1,2_2_6_1,2_2_6_2,2_3_6_2,2_2_5_2}"
 for v in "${FORMS[@]}"; do
  set -- ${v//_/ }
  T=$1_$2_$3_$4_${5:-0}_${6:-1}_${7:-3}_r$rep
  LMOSEM_ZLIST=$1 LMOSEM_ZFINE=$2 LMOSEM_ZFUSED_MODE=$3 LMOSEM_ZOVER=$4 LMOSEM_ZWIN=${5:-0} LMOSEM_ZMERGE=${6:-1} LMOSEM_ZMED=${7:-3} timeout 300 python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_$T.json 2>$O/b_$T.err
  python -c "import json;d=json.load(open('$O/b_$T.json'));print('C4 zlist=$1 zfine=$2 mode=$3 zover=$4 zwin=${5:-0} zmerge=${6:-1} zmed=${7:-3}', round(d['ms_per_step'],3), d['phase_ms_per_step'].get('project'))" 2>&1 | tail -1
 done
done
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sector_hit_rate.pct,sm__inst_executed.sum
IFS=',' read -ra NFORMS <<< "${ZAB_NCU:-0_2_1,2_2_1,2_2_2}"
for v in "${NFORMS[@]}"; do set -- ${v//_/ }
LMOSEM_ZLIST=$1 LMOSEM_ZFINE=$2 LMOSEM_ZOVER=$3 ncu --clock-control none --cache-control none --metrics $M -k regex:"k_project|k_zclass" -s 40 -c 40 --csv --log-file $O/ncu_z$1_$2_$3.csv python bench.py --config C4 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e > /dev/null 2>&1
done
