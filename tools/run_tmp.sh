mkdir -p gpurun_out
SWDUAL_LIB=build/variants/s32.so PROF_WORKLOAD=c3 PROF_NDB=100000 PROF_REPS=1 timeout 600 ncu --set full --import-source on -k regex:inter_kernel -c 1 -o gpurun_out/full_s32 -f python tools/prof_one.py > gpurun_out/full_s32.log 2>&1
bash tools/gpu_ab_libs.sh v5 s32 pk pk@pack_queries=0
