mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/r1_smi.txt
timeout 1200 python -m pytest tests -x -q -m gpu > gpurun_out/r1_tests.log 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r1_smoke.log 2>&1
timeout 600 python bench.py > gpurun_out/r1_bench_c3.json 2> gpurun_out/r1_bench_c3.err
timeout 600 python bench.py --workload c4 --no-cpu-baseline > gpurun_out/r1_bench_c4.json 2> gpurun_out/r1_bench_c4.err
timeout 600 python bench.py --workload c2 --no-cpu-baseline > gpurun_out/r1_bench_c2.json 2> gpurun_out/r1_bench_c2.err
