#!/bin/bash
T=${1:-r2f}; mkdir -p gpurun_out
PROF_WORKLOAD=c1 PROF_REPS=2 timeout 600 ncu --set full --clock-control none --import-source on \
  -k regex:short_kernel --launch-skip 1 -c 1 -o gpurun_out/${T}_full_c1 -f python tools/prof_one.py > gpurun_out/${T}_full_c1.log 2>&1
PROF_WORKLOAD=c4 PROF_REPS=1 timeout 900 ncu --set full --clock-control none --import-source on \
  -k regex:rescore -c 1 -o gpurun_out/${T}_full_c4_rescore -f python tools/prof_one.py > gpurun_out/${T}_full_c4_rescore.log 2>&1
python - > gpurun_out/${T}_c4_ovf.txt 2>&1 <<'PY'
import sys, os, torch
sys.path.insert(0, os.getcwd())
import swgen, paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
c = swgen.make_config("c4")
h = sw.Handle(0, timing=True)
db = h.load_db(c["dcodes"], c["doff"])
for _ in range(2):
    out = h.search(c["qcodes"], c["qoff"], db, sw.blosum62(), 10, 2)
    torch.cuda.synchronize()
    print(h.last_stats())
import numpy as np
o = out.cpu().numpy(); print("scores > 32756:", int((o > 32756).sum()), [int(x) for x in np.sort(o.ravel())[-12:]])
PY
echo done
