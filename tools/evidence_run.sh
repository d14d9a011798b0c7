#!/bin/bash
# One GPU call that refreshes the round's committed evidence (run under gpurun).
# Outputs land in gpurun_out/ev_*; tools/ncu_summary.py turns the ncu files into profiles/ summaries.
set -x
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/ev_smi.txt
# 0. the bench lines (default = config 3, N=1; plus configs 1, 2, 4)
python bench.py > gpurun_out/ev_bench_c3.json 2> gpurun_out/ev_bench_c3.err
for w in c1 c2 c4; do python bench.py --workload $w --no-cpu-baseline > gpurun_out/ev_bench_$w.json 2> gpurun_out/ev_bench_$w.err; done
python bench.py --impl reference --steps 2 --warmup 3 > gpurun_out/ev_bench_ref.json 2> gpurun_out/ev_bench_ref.err
# 1. launch list of one bench step (serialised, cold-cache: compare shares, not absolutes)
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/ev_launches.csv \
    python bench.py --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/ev_launches_bench.log 2>&1
# 2. DRAM traffic of the scoring kernel (one launch of each bench workload)
for w in c2 c3 c4; do
ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
    -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/ev_traffic_$w.csv \
    python bench.py --workload $w --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/ev_traffic_$w.log 2>&1
done
# 3. full captures of the scoring kernel: config 3 (whole workload) and config 4
PROF_WORKLOAD=c3 PROF_REPS=1 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/ev_full_c3 -f \
    python tools/prof_one.py > gpurun_out/ev_full_c3.log 2>&1
PROF_WORKLOAD=c4 PROF_REPS=1 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/ev_full_c4 -f \
    python tools/prof_one.py > gpurun_out/ev_full_c4.log 2>&1
# 4. the multi-rank bench path, functionally (2 ranks share GPU 0 over gloo) with sampled verification
python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 \
    bench.py --gpus 2 --dist-backend gloo --n-db 60000 --steps 2 --warmup 3 --no-cpu-baseline --e2e-steps 1 \
    --verify 300 > gpurun_out/ev_2rank_gloo.json 2> gpurun_out/ev_2rank_gloo.err
# 5. config 5 on one GPU with sampled parity
timeout 900 python tools/c5_run.py > gpurun_out/ev_c5.json 2> gpurun_out/ev_c5.err
