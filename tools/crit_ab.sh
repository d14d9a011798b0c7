#!/bin/bash
mkdir -p gpurun_out; TAG=$1
for pct in 35 70 100 150; do
  for mn in 16384 4096; do
    SWDUAL_OPTS=crit_pct=$pct,crit_min_steps=$mn timeout 600 python tools/shard_probe.py 2 >> gpurun_out/${TAG}_shard.jsonl 2>&1
    SWDUAL_OPTS=crit_pct=$pct,crit_min_steps=$mn timeout 600 python tools/shard_probe.py 8 >> gpurun_out/${TAG}_shard.jsonl 2>&1
  done
  SWDUAL_OPTS=crit_pct=$pct timeout 600 python bench.py --no-cpu-baseline --e2e-steps 0 --steps 3 --warmup 2 > gpurun_out/${TAG}_c3_pct$pct.json 2>/dev/null
done
echo done
