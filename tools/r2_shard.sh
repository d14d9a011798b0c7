#!/bin/bash
mkdir -p gpurun_out; TAG=$1
for k in 2 4 8; do timeout 600 python tools/shard_probe.py $k >> gpurun_out/${TAG}_shard.jsonl 2>&1; done
timeout 600 python tools/shard_probe.py 8 8 pair >> gpurun_out/${TAG}_shard.jsonl 2>&1
timeout 600 python tools/shard_probe.py 8 32 pair >> gpurun_out/${TAG}_shard.jsonl 2>&1
echo done
