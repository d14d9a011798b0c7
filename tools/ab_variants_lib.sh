#!/bin/bash
# A/B of library builds (build/variants/NAME.so via SWDUAL_LIB; "base" = in-tree) per workload.
# usage: tools/ab_variants_lib.sh TAG "c4 c2" base lag16 ...
mkdir -p gpurun_out; TAG=$1; WLS=$2; shift 2
for w in $WLS; do
  for v in "$@"; do
    lib=""; [ "$v" != base ] && lib="build/variants/$v.so"
    SWDUAL_LIB=$lib timeout 600 python bench.py --workload $w --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 3 \
      > gpurun_out/${TAG}_${v}_$w.json 2> gpurun_out/${TAG}_${v}_$w.err
    echo "$w $v $(python -c "import json; d=json.load(open('gpurun_out/${TAG}_${v}_$w.json')); print(d['value'], d['roofline']['frac'], d['detail'])" 2>&1)" >> gpurun_out/${TAG}.txt
  done
done
echo done
