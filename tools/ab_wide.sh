# same-box A/B of the wide single-query profile (option wide_profile: IMAD pair build instead of PRMT)
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "wide or single_query_profile_copies or resident or small_random or pairing or swissprot or geometry" > gpurun_out/wide_parity.log 2>&1; echo EXIT $? >> gpurun_out/wide_parity.log
for i in 1 2; do
  for wd in 1 0; do
    SWDUAL_OPTS=wide_profile=$wd timeout 300 python bench.py --workload c2 --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('c2', 'wide=$wd', d['value'], d['ms_per_step'], d['roofline'].get('frac'), d['e2e']['value'], d['clocks']['sm_mhz'])" >> gpurun_out/ab_wide.txt
  done
done
for wd in 1 0; do
  SWDUAL_OPTS=wide_profile=$wd timeout 300 python bench.py --workload c1 --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('c1', 'wide=$wd', d['value'], d['ms_per_step'])" >> gpurun_out/ab_wide.txt
done
SWDUAL_OPTS=wide_profile=1 PROF_WORKLOAD=c2 PROF_REPS=1 timeout 300 ncu --clock-control none --metrics sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_active,sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active,l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum,gpu__time_duration.sum -k regex:inter_kernel -c 1 --csv python tools/prof_one.py 2>/dev/null | grep -E "pipe|conflicts|duration" | awk -F'","' '{print "wide=1 ncu", $(NF-2), $NF}' >> gpurun_out/ab_wide.txt
