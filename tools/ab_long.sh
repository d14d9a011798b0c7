#!/bin/bash
# C4 / C2 with long-link variants (build/variants/*.so via SWDUAL_LIB)
mkdir -p gpurun_out; TAG=$1
for v in base lag16 lag0 prog4; do
  lib=""; [ "$v" != base ] && lib="build/variants/$v.so"
  for w in c4 c2; do
    SWDUAL_LIB=$lib timeout 600 python bench.py --workload $w --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 2 \
      > gpurun_out/${TAG}_${v}_$w.json 2> gpurun_out/${TAG}_${v}_$w.err
  done
done
echo done
