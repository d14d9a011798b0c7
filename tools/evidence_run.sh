#!/bin/bash
# One GPU call that refreshes the round's committed evidence (run under gpurun).
set -x
mkdir -p gpurun_out
# 1. launch list of one bench step (serialised, cold-cache: compare shares, not absolutes)
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/ev_launches.csv \
    python bench.py --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/ev_launches_bench.log 2>&1
# 2. DRAM traffic of the scoring kernel (one launch of the bench workload)
ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
    -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/ev_traffic_c3.csv \
    python bench.py --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/ev_traffic.log 2>&1
ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
    -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/ev_traffic_c2.csv \
    python bench.py --workload c2 --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/ev_traffic2.log 2>&1
# 3. the multi-rank bench path, functionally (2 ranks share GPU 0 over gloo) with sampled verification
python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 \
    bench.py --gpus 2 --dist-backend gloo --n-db 60000 --steps 2 --warmup 1 --no-cpu-baseline --e2e-steps 1 \
    --verify 300 > gpurun_out/ev_2rank_gloo.json 2> gpurun_out/ev_2rank_gloo.err
# 4. config 5 on one GPU with sampled parity
timeout 900 python tools/c5_run.py > gpurun_out/ev_c5.json 2> gpurun_out/ev_c5.err
