#!/bin/bash
# GPU tests (optional -k filter) then bench lines for a list of "workload:geom" specs.
# usage: tools/r2_ab.sh TAG "pytest -k expr or empty" "c3: c3:4,32 c4: c2:"
TAG=$1; K=$2; SPECS=$3
mkdir -p gpurun_out
if [ "$K" != "none" ]; then
  if [ -n "$K" ]; then timeout 2400 python -m pytest tests -q -m gpu -x --timeout=600 --timeout-method=thread -k "$K" > gpurun_out/${TAG}_tests.log 2>&1
  else timeout 2400 python -m pytest tests -q -m gpu --timeout=600 --timeout-method=thread > gpurun_out/${TAG}_tests.log 2>&1; fi
fi
for spec in $SPECS; do
  w=${spec%%:*}; g=${spec#*:}
  extra=""; [ -n "$g" ] && extra="--force-geom $g"
  timeout 900 python bench.py --workload $w --no-cpu-baseline --e2e-steps 0 --steps 5 --warmup 3 $extra \
    > gpurun_out/${TAG}_bench_${w}_${g/,/x}.json 2> gpurun_out/${TAG}_bench_${w}_${g/,/x}.err
done
echo done
