# A/B of alternative builds (SWDUAL_LIB) and geometries on the bench workloads
run() { # variant geom tag
  SWDUAL_LIB=build/variants/$1.so python bench.py --no-cpu-baseline --steps 3 --warmup 2 --e2e-steps 0 ${2:+--force-geom $2} > gpurun_out/ab_$3.json 2>&1
}
run C "" C_auto
run D "" D_auto
run D 4,16 D_4_16
run D 4,20 D_4_20
run C 4,28 C_4_28
run C 8,24 C_8_24
