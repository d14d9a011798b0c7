mkdir -p gpurun_out
bash tools/gpu_ab_libs.sh v10 du2 cd0 cd1 cd2
for v in cd1 cd2; do
SWDUAL_LIB=build/variants/$v.so ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:inter_kernel -c 1 --csv --log-file gpurun_out/traffic_$v.csv python bench.py --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/traffic_$v.log 2>&1
done
