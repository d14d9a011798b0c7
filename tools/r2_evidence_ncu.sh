#!/bin/bash
# Round-2 end-of-round evidence, part 2: ncu --set full of the dominant kernels (summarised on the box),
# C5 on one GPU and through the 2-rank path.
T=${1:-r2z}; mkdir -p gpurun_out
PROF_WORKLOAD=c3 PROF_NDB=100000 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:short_kernel -c 1 -o gpurun_out/${T}_full_c3sub -f python tools/prof_one.py > gpurun_out/${T}_full_c3sub.log 2>&1
PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:long_kernel -c 1 -o gpurun_out/${T}_full_c4 -f python tools/prof_one.py > gpurun_out/${T}_full_c4.log 2>&1
PROF_WORKLOAD=c2 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:combined -c 1 -o gpurun_out/${T}_full_c2 -f python tools/prof_one.py > gpurun_out/${T}_full_c2.log 2>&1
# summaries on the box (the .ncu-rep files exceed gpurun's 64 MiB copy-back limit)
for r in c3sub c4 c2; do
  if [ -f gpurun_out/${T}_full_$r.ncu-rep ]; then
    python tools/ncu_summary.py full gpurun_out/${T}_full_$r.ncu-rep gpurun_out/${T}_ncu_$r.json > /dev/null 2>&1
    ncu -i gpurun_out/${T}_full_$r.ncu-rep --page source --csv --print-source sass > gpurun_out/${T}_src_$r.csv 2>/dev/null
    rm -f gpurun_out/${T}_full_$r.ncu-rep
  fi
done
timeout 1800 python bench.py --workload c5 --steps 1 --warmup 1 --e2e-steps 0 --no-cpu-baseline > gpurun_out/${T}_bench_c5.json 2> gpurun_out/${T}_bench_c5.err
bash tools/c5_multirank.sh ${T}
echo done
