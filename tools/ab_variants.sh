run() { # variant geom tag [workload]
  SWDUAL_LIB=build/variants/$1.so python bench.py --no-cpu-baseline --steps 3 --warmup 2 --e2e-steps 0 ${4:+--workload $4} ${2:+--force-geom $2} > gpurun_out/ab_$3.json 2>&1
}
run I "" I_auto
run C "" C_auto5
run I "" I_c2 c2
SWDUAL_LIB=build/variants/I.so python tools/c3_probe.py > gpurun_out/c3_probe_I.jsonl 2>&1
SWDUAL_LIB=build/variants/I.so python -m pytest tests -x -q -m gpu 2>&1 | tail -2 > gpurun_out/ab_tests_I.log
