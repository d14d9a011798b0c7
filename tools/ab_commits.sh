#!/bin/bash
# A/B of earlier commits (worktrees under abwt/) against HEAD: bench lines per workload.
# usage: tools/ab_commits.sh TAG "c4 c2 c3" commit1 commit2 ...
mkdir -p gpurun_out; TAG=$1; WLS=$2; shift 2
ROOT=$(pwd)
for w in $WLS; do
  for c in "$@" HEAD; do
    d=$ROOT; [ "$c" != HEAD ] && d=$ROOT/abwt/$c
    (cd $d && timeout 600 python bench.py --workload $w --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 3 > $ROOT/gpurun_out/${TAG}_${c}_$w.json 2>$ROOT/gpurun_out/${TAG}_${c}_$w.err)
    echo "$w $c $(python -c "import json; d=json.load(open('$ROOT/gpurun_out/${TAG}_${c}_$w.json')); print(d['value'], d['roofline']['frac'], d['detail'])" 2>&1)" >> gpurun_out/${TAG}.txt
  done
done
echo done
