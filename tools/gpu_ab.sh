# A/B of handle options on one GPU: bash tools/gpu_ab.sh TAG "opts1" "opts2" ... (workload via WL env, default c3)
mkdir -p gpurun_out
WL=${WL:-c3}
tag=$1; shift
i=0
for o in "$@"; do
  SWDUAL_OPTS=$o timeout 600 python bench.py --workload $WL --no-cpu-baseline --steps ${STEPS:-3} --warmup 3 --e2e-steps 0 > gpurun_out/ab_${tag}_${WL}_$i.json 2> gpurun_out/ab_${tag}_${WL}_$i.err
  echo "$o -> $(python -c "import json,sys; d=json.load(open('gpurun_out/ab_${tag}_${WL}_$i.json')); print(d['value'], d['roofline']['frac'])" 2>&1)" >> gpurun_out/ab_${tag}.txt
  i=$((i+1))
done
