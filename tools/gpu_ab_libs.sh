# Same-box A/B of library builds: WL=c3 bash tools/gpu_ab_libs.sh TAG lib1 lib2@opt=v,opt2=v ...
# (build/variants/<lib>.so; "@..." sets SWDUAL_OPTS handle options for that arm)
mkdir -p gpurun_out
WL=${WL:-c3}
tag=$1; shift
for rep in 1 2; do
for v in "$@"; do
  lib=${v%%@*}; opts=""; [[ "$v" == *@* ]] && opts=${v#*@}
  out=gpurun_out/abl_${tag}_${WL}_${lib}_${rep}
  SWDUAL_OPTS=$opts SWDUAL_LIB=build/variants/$lib.so timeout 600 python bench.py --workload $WL --no-cpu-baseline --steps ${STEPS:-3} --warmup 3 --e2e-steps 0 ${EXTRA:-} > $out.json 2> $out.err
  echo "$WL $v rep$rep -> $(python -c "import json; d=json.load(open('$out.json')); print(d['value'], d['roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1)" >> gpurun_out/abl_${tag}.txt
done
done
