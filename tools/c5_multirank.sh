#!/bin/bash
# C5 through the multi-rank path (2 ranks sharing one GPU over gloo; functional) and on one GPU
mkdir -p gpurun_out; TAG=$1
free -g > gpurun_out/${TAG}_mem.txt; nproc >> gpurun_out/${TAG}_mem.txt
timeout 2400 python -m torch.distributed.run --nnodes=1 --nproc-per-node=2 --master-addr=127.0.0.1 --master-port=29731 \
  bench.py --gpus 2 --dist-backend gloo --workload c5 --steps 1 --warmup 1 --e2e-steps 0 --verify 300 --no-cpu-baseline \
  > gpurun_out/${TAG}_c5_2rank.json 2> gpurun_out/${TAG}_c5_2rank.err
echo done
