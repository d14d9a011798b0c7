set -x
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q > gpurun_out/res_parity.log 2>&1; echo EXIT $? >> gpurun_out/res_parity.log
for w in c2 c1 c3 t5hom c2; do
  for r in 1 0; do
    SWDUAL_OPTS=resident_strips=$r timeout 300 python bench.py --workload $w --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$w', 'res=$r', d['value'], d['ms_per_step'], d['roofline'].get('frac'), d['e2e']['value'])" >> gpurun_out/ab_res.txt
  done
done
