#!/bin/bash
# Round-2 GPU check: selected GPU tests, smoke, one C3 bench line.
# usage: tools/r2_check.sh TAG "pytest -k expression"
TAG=${1:-r2}
K=${2:-}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv > gpurun_out/${TAG}_smi.txt
if [ -n "$K" ]; then
  timeout 2400 python -m pytest tests -q -m gpu -k "$K" > gpurun_out/${TAG}_tests.log 2>&1
else
  timeout 2400 python -m pytest tests -q -m gpu > gpurun_out/${TAG}_tests.log 2>&1
fi
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${TAG}_smoke.log 2>&1
timeout 900 python bench.py > gpurun_out/${TAG}_bench_c3.json 2> gpurun_out/${TAG}_bench_c3.err
echo done
