#!/bin/bash
# Round-2 end-of-round evidence, part 1: bench lines (C3 default with the cpu_baseline, C4, C2,
# C1, Table V), the oracle arm, the C3 launch list, smoke, the GPU suite (part 2:
# tools/r2_evidence_ncu.sh).
T=${1:-r2z}; mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/${T}_smi.txt
timeout 900 python bench.py > gpurun_out/${T}_bench_c3.json 2> gpurun_out/${T}_bench_c3.err
for w in c4 c2 c1 t5hom t5het; do
  timeout 900 python bench.py --workload $w --no-cpu-baseline > gpurun_out/${T}_bench_$w.json 2> gpurun_out/${T}_bench_$w.err
done
timeout 900 python bench.py --impl reference --steps 2 --warmup 3 > gpurun_out/${T}_bench_ref.json 2> gpurun_out/${T}_bench_ref.err
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/${T}_launches_c3.csv \
  python bench.py --steps 1 --warmup 1 --no-cpu-baseline --e2e-steps 0 > gpurun_out/${T}_launches_c3.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
timeout 3000 python -m pytest tests -q -m gpu -rf --timeout=1200 > gpurun_out/${T}_gpu_tests.txt 2>&1
echo done
