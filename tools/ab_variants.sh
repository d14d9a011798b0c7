# A/B of alternative builds (SWDUAL_LIB) and geometries on the bench workloads
run() { # variant geom tag [workload]
  SWDUAL_LIB=build/variants/$1.so python bench.py --no-cpu-baseline --steps 3 --warmup 2 --e2e-steps 0 ${4:+--workload $4} ${2:+--force-geom $2} > gpurun_out/ab_$3.json 2>&1
}
SWDUAL_LIB=build/variants/E.so python -m pytest tests -x -q -m gpu -k "geometry or pairing or intra or small or c1" 2>&1 | tail -2 > gpurun_out/ab_tests_E.log
run C "" C_auto
run E "" E_auto
run E 4,24 E_4_24
run E 8,24 E_8_24
run E 4,20 E_4_20
run E "" E_c2 c2
run C "" C_c2 c2
