#!/bin/bash
# A/B of the round-1 build (worktree old_r1/, commit fd8a28d) against HEAD on C4 / C2
mkdir -p gpurun_out; TAG=$1
ROOT=$(pwd)
for w in c4 c2; do
  (cd old_r1 && timeout 600 python bench.py --workload $w --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 2 > $ROOT/gpurun_out/${TAG}_old_$w.json 2>$ROOT/gpurun_out/${TAG}_old_$w.err)
  timeout 600 python bench.py --workload $w --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 2 > gpurun_out/${TAG}_new_$w.json 2>gpurun_out/${TAG}_new_$w.err
done
(cd old_r1 && PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full -k regex:inter_kernel -c 1 -o $ROOT/gpurun_out/${TAG}_old_full_c4 -f python tools/prof_one.py > $ROOT/gpurun_out/${TAG}_old_full_c4.log 2>&1)
PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full --import-source on -k regex:long_kernel -c 1 -o gpurun_out/${TAG}_new_full_c4 -f python tools/prof_one.py > gpurun_out/${TAG}_new_full_c4.log 2>&1
echo done
