#!/bin/bash
# Re-entry GPU check of HEAD: full GPU suite, smoke, bench lines C3 (default), C4, C2, C1.
T=${1:-r2b}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/${T}_smi.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
timeout 900 python bench.py > gpurun_out/${T}_bench_c3.json 2> gpurun_out/${T}_bench_c3.err
for w in c4 c2 c1; do
  timeout 600 python bench.py --workload $w --no-cpu-baseline > gpurun_out/${T}_bench_$w.json 2> gpurun_out/${T}_bench_$w.err
done
timeout 3000 python -m pytest tests -q -m gpu --timeout=900 --timeout-method=thread > gpurun_out/${T}_gpu_tests.txt 2>&1
echo done
