mkdir -p gpurun_out
for g in "4,24" "8,24" "8,16" "4,28"; do
  G=${g%,*}; R=${g#*,}
  timeout 600 python bench.py --workload c3 --no-cpu-baseline --steps 3 --warmup 3 --e2e-steps 0 --force-geom $g > gpurun_out/geo_${G}_${R}.json 2>/dev/null
  timeout 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:inter_kernel -c 1 --csv \
     python bench.py --workload c3 --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 --force-geom $g > gpurun_out/geo_${G}_${R}.csv 2>&1
done
