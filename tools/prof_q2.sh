#!/bin/bash
# ncu full captures: the query-pair kernel on a C3 slice, the long kernel on C4; launch lists of c2/c4
mkdir -p gpurun_out
TAG=$1
for w in c2 c4; do
  timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/${TAG}_launches_${w}.csv \
    python bench.py --workload $w --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/${TAG}_launches_${w}.log 2>&1
done
PROF_WORKLOAD=c3 PROF_NDB=60000 PROF_REPS=1 timeout 900 ncu --set full --import-source on -k regex:short_kernel_q2 -c 1 \
  -o gpurun_out/${TAG}_full_c3sub -f python tools/prof_one.py > gpurun_out/${TAG}_full_c3sub.log 2>&1
PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full --import-source on -k regex:long_kernel -c 1 \
  -o gpurun_out/${TAG}_full_c4 -f python tools/prof_one.py > gpurun_out/${TAG}_full_c4.log 2>&1
echo done
