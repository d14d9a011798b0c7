mkdir -p gpurun_out
for v in base inp1; do
  SWDUAL_LIB=build/variants/$v.so PROF_WORKLOAD=c3 PROF_NDB=100000 PROF_REPS=1 timeout 600 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/full_$v -f python tools/prof_one.py > gpurun_out/full_$v.log 2>&1
done
