#!/bin/bash
# launch lists (per-kernel device times, serialised) and one full ncu capture
# usage: tools/r2_prof.sh TAG "c2 c4" KERNEL_REGEX WORKLOAD_FOR_FULL
TAG=$1; WL=$2; KRE=$3; WF=$4
mkdir -p gpurun_out
for w in $WL; do
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/${TAG}_launches_${w}.csv \
    python bench.py --workload $w --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/${TAG}_launches_${w}.log 2>&1
done
if [ -n "$KRE" ]; then
  PROF_WORKLOAD=$WF PROF_REPS=1 timeout 1200 ncu --set full --import-source on -k regex:$KRE -c 1 \
    -o gpurun_out/${TAG}_full_${WF} -f python tools/prof_one.py > gpurun_out/${TAG}_full_${WF}.log 2>&1
fi
echo done
