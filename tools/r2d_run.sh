#!/bin/bash
# Benches (C3 default line incl. cpu_baseline, C4, C2, C1), launch lists C3/C4, full GPU suite, smoke.
T=${1:-r2d}; mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/${T}_smi.txt
timeout 900 python bench.py > gpurun_out/${T}_bench_c3.json 2> gpurun_out/${T}_bench_c3.err
for w in c4 c2 c1; do
  timeout 600 python bench.py --workload $w --no-cpu-baseline > gpurun_out/${T}_bench_$w.json 2> gpurun_out/${T}_bench_$w.err
done
for w in c3 c4; do
  timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/${T}_launches_$w.csv \
    python bench.py --workload $w --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/${T}_launches_$w.log 2>&1
done
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
timeout 3000 python -m pytest tests -q -m gpu -rf --timeout=1200 > gpurun_out/${T}_gpu_tests.txt 2>&1
echo done
