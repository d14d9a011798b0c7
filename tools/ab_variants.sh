run() { # variant opts tag workload
  SWDUAL_OPTS=$2 SWDUAL_LIB=build/variants/$1.so python bench.py --no-cpu-baseline --steps 3 --warmup 2 --e2e-steps 0 --workload $4 > gpurun_out/ab_$3.json 2>&1
}
SWDUAL_LIB=build/variants/N.so python -m pytest tests -x -q -m gpu 2>&1 | tail -2 > gpurun_out/ab_tests_N.log
for w in c3 c2 c4; do run N "" N_$w $w; done
