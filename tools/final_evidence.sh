#!/bin/bash
# Round-end evidence in one GPU call (outputs gpurun_out/fe_*).
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/fe_smi.txt
timeout 1500 python -m pytest tests -q -m gpu > gpurun_out/fe_tests.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/fe_smoke.log 2>&1
timeout 600 python bench.py > gpurun_out/fe_bench_c3.json 2> gpurun_out/fe_bench_c3.err
for w in c1 c2 c4 t5hom t5het; do timeout 900 python bench.py --workload $w --no-cpu-baseline > gpurun_out/fe_bench_$w.json 2> gpurun_out/fe_bench_$w.err; done
timeout 600 python bench.py --impl reference --steps 2 --warmup 3 > gpurun_out/fe_bench_ref.json 2> gpurun_out/fe_bench_ref.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/fe_launches.csv \
    python bench.py --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/fe_launches_bench.log 2>&1
for w in c3 c2 c4; do
timeout 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
    -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/fe_traffic_$w.csv \
    python bench.py --workload $w --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/fe_traffic_$w.log 2>&1
done
PROF_WORKLOAD=c3 PROF_NDB=100000 PROF_REPS=1 timeout 1200 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/fe_full_c3sub -f \
    python tools/prof_one.py > gpurun_out/fe_full_c3sub.log 2>&1
PROF_WORKLOAD=c4 PROF_REPS=1 timeout 1200 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/fe_full_c4 -f \
    python tools/prof_one.py > gpurun_out/fe_full_c4.log 2>&1
timeout 1200 python tools/c5_run.py > gpurun_out/fe_c5.json 2> gpurun_out/fe_c5.err
echo done
