for v in A B C; do
  SWDUAL_LIB=build/variants/$v.so python bench.py --no-cpu-baseline --steps 3 --warmup 2 --e2e-steps 0 > gpurun_out/ab_$v.json 2>&1
  SWDUAL_LIB=build/variants/$v.so python bench.py --workload c2 --no-cpu-baseline --steps 5 --warmup 3 --e2e-steps 0 > gpurun_out/ab_c2_$v.json 2>&1
done
SWDUAL_LIB=build/variants/C.so ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/ab_traffic_C.csv python bench.py --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > /dev/null 2>&1
