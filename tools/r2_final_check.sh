#!/bin/bash
# Final HEAD check: smoke, GPU suite, default bench line, DPX microbenchmark (fixed lone-max probe).
T=${1:-r2w}; mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
timeout 900 python bench.py > gpurun_out/${T}_bench_c3.json 2> gpurun_out/${T}_bench_c3.err
timeout 300 ./tools/dpx_microbench > gpurun_out/${T}_dpx_microbench.jsonl 2>&1
timeout 3000 python -m pytest tests -q -m gpu -rf --timeout=1200 > gpurun_out/${T}_gpu_tests.txt 2>&1
echo done
