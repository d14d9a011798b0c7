# same-box A/B of option pack_long (several long pairs per CTA when a query has fewer intra-task strips than warps)
timeout 300 python -m pytest tests/test_gpu_parity.py -x -q -k "long or c4 or intra" > gpurun_out/pl_parity.log 2>&1; echo EXIT $? >> gpurun_out/pl_parity.log
for i in 1 2; do
  for pl in 1 0; do
    SWDUAL_OPTS=pack_long=$pl timeout 300 python bench.py --workload c4 --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('c4', 'pack_long=$pl', d['value'], d['ms_per_step'], d['roofline'].get('frac'))" >> gpurun_out/ab_pl.txt
  done
done
for pl in 1 0; do
  SWDUAL_OPTS=pack_long=$pl timeout 300 python bench.py --workload c3 --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('c3', 'pack_long=$pl', d['value'], d['ms_per_step'], d['roofline'].get('frac'))" >> gpurun_out/ab_pl.txt
done
