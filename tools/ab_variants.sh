run() { # variant opts tag workload
  SWDUAL_OPTS=$2 SWDUAL_LIB=build/variants/$1.so python bench.py --no-cpu-baseline --steps 3 --warmup 3 --e2e-steps 0 --workload $4 > gpurun_out/ab_$3.json 2>&1
}
SWDUAL_LIB=build/variants/O.so timeout 900 python -m pytest tests -x -q -m gpu 2>&1 | tail -2 > gpurun_out/ab_tests_O.log
run O "" O_c4 c4
SWDUAL_LIB=build/variants/O.so timeout 300 python tools/c4_probe.py > gpurun_out/c4_probe_O.txt 2>&1
