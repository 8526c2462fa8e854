#!/bin/bash
# A/B of the z-slab passes' CTA shape at C4 (variants/liblmosem_z<T>b<B>.so; default 128 x 7).
O=gpurun_out/slab_shape_ab
mkdir -p $O
for rep in 1 2; do
 for v in default z224b4 z64b14 z256b3; do
  if [ $v = default ]; then L=""; else L=variants/liblmosem_$v.so; fi
  LMOSEM_LIB=$L python bench.py --config C4 --steps 10 --no-cpu-baseline --no-e2e > $O/b_${v}_r$rep.json 2>/dev/null
  python -c "import json;d=json.load(open('$O/b_${v}_r$rep.json'));print('$v', round(d['ms_per_step'],3), d['clocks']['reasons'])"
 done
done
