#!/bin/bash
# Long-item latency probe; DRAM traffic of the dominant kernel per workload (one launch, ncu).
T=${1:-r2e}; mkdir -p gpurun_out
timeout 600 python tools/long_item_probe.py > gpurun_out/${T}_long_probe.jsonl 2> gpurun_out/${T}_long_probe.err
for spec in c3:short_kernel c2:combined_m0_kernel c4:long_kernel c1:short_kernel; do
  w=${spec%%:*}; k=${spec#*:}
  timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none \
    -k regex:$k -c 1 --csv --log-file gpurun_out/${T}_traffic_$w.csv \
    python bench.py --workload $w --steps 1 --warmup 0 --no-cpu-baseline --e2e-steps 0 > gpurun_out/${T}_traffic_$w.log 2>&1
done
echo done
