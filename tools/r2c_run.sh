#!/bin/bash
# Post-revert check: bench lines, C3 long-pair rule A/B, ncu full captures (C3 short, C4 long old/new).
T=${1:-r2c}; mkdir -p gpurun_out; ROOT=$(pwd)
for w in c3 c4 c2 c1; do
  timeout 600 python bench.py --workload $w --no-cpu-baseline --steps 5 --warmup 3 > gpurun_out/${T}_bench_$w.json 2> gpurun_out/${T}_bench_$w.err
done
for o in "crit_pct=70" "crit_pct=150" "crit_pct=300"; do
  SWDUAL_OPTS=$o timeout 600 python bench.py --workload c3 --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 3 > gpurun_out/${T}_c3_$o.json 2> gpurun_out/${T}_c3_$o.err
done
PROF_WORKLOAD=c3 PROF_NDB=100000 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:short_kernel -c 1 -o gpurun_out/${T}_full_c3sub -f python tools/prof_one.py > gpurun_out/${T}_full_c3sub.log 2>&1
PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:long_kernel -c 1 -o gpurun_out/${T}_full_c4 -f python tools/prof_one.py > gpurun_out/${T}_full_c4.log 2>&1
(cd abwt/9267477 && PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:inter_kernel -c 1 -o $ROOT/gpurun_out/${T}_full_c4_old -f python tools/prof_one.py > $ROOT/gpurun_out/${T}_full_c4_old.log 2>&1)
echo done
