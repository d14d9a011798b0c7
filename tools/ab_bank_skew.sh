# same-box A/B of the bank-skewed single-query profile copies (option bank_skew)
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "single_query_profile_copies or resident or every_geometry or pairing or swissprot" > gpurun_out/skew_parity.log 2>&1; echo EXIT $? >> gpurun_out/skew_parity.log
for i in 1 2; do
  for sk in 1 0; do
    SWDUAL_OPTS=bank_skew=$sk timeout 300 python bench.py --workload c2 --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('c2', 'bank_skew=$sk', d['value'], d['ms_per_step'], d['roofline'].get('frac'), d['e2e']['value'], d['clocks']['sm_mhz'])" >> gpurun_out/ab_skew.txt
  done
done
for sk in 1 0; do
  SWDUAL_OPTS=bank_skew=$sk timeout 300 python bench.py --workload c2 --force-geom 16,24 --no-cpu-baseline 2>/dev/null | python -c "import sys,json; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('c2 G16R24', 'bank_skew=$sk', d['value'], d['ms_per_step'])" >> gpurun_out/ab_skew.txt
done
for sk in 1 0; do
  SWDUAL_OPTS=bank_skew=$sk PROF_WORKLOAD=c2 PROF_REPS=1 timeout 300 ncu --clock-control none --metrics l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum,smsp__inst_executed_op_shared_ld.sum,gpu__time_duration.sum -k regex:inter_kernel -c 1 --csv python tools/prof_one.py 2>/dev/null | grep -E "bank_conflicts|shared_ld|duration" | sed "s/^/bank_skew=$sk /" >> gpurun_out/ab_skew.txt
done
