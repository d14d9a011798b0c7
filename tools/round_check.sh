#!/bin/bash
# One GPU call: GPU tests, smoke, bench lines (c3 default + c2/c4), launch list, c3 traffic, c3 full ncu.
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/rc_smi.txt
timeout 1200 python -m pytest tests -x -q -m gpu > gpurun_out/rc_tests.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/rc_smoke.log 2>&1
timeout 600 python bench.py > gpurun_out/rc_bench_c3.json 2> gpurun_out/rc_bench_c3.err
for w in c2 c4 c1; do timeout 600 python bench.py --workload $w --no-cpu-baseline > gpurun_out/rc_bench_$w.json 2> gpurun_out/rc_bench_$w.err; done
timeout 600 python bench.py --impl reference --steps 2 --warmup 3 > gpurun_out/rc_bench_ref.json 2> gpurun_out/rc_bench_ref.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/rc_launches.csv \
    python bench.py --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/rc_launches_bench.log 2>&1
timeout 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
    -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/rc_traffic_c3.csv \
    python bench.py --workload c3 --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/rc_traffic_c3.log 2>&1
PROF_WORKLOAD=c3 PROF_REPS=1 timeout 900 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/rc_full_c3 -f \
    python tools/prof_one.py > gpurun_out/rc_full_c3.log 2>&1
echo done
