"""Per-rank device time of the k-GPU placement of C3, run rank after rank on one GPU
(the layout the multi-GPU path uses), vs the placement model; options via SWDUAL_OPTS.
  python tools/shard_probe.py K [n_shards]"""
import json, os, sys
import numpy as np
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402
from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist  # noqa: E402

k = int(sys.argv[1]); S = int(sys.argv[2]) if len(sys.argv) > 2 else k
mode = sys.argv[3] if len(sys.argv) > 3 else "shard"
c = swgen.make_config("c3")
ql = np.diff(c["qoff"])
sh = dist.shard_cut(c["doff"], S)
res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
plan = dist.place_shards(ql, sh, res, k) if mode == "shard" else dist.place(ql, sh, res, k)
with sw.Handle(0, timing=True) as h:
    for kv in filter(None, os.environ.get("SWDUAL_OPTS", "").split(",")):
        h.set_option(kv.split("=")[0], int(kv.split("=")[1]))
    dbs = {s: h.load_db(*dist.subset(c["dcodes"], c["doff"], sh[s])) for s in range(len(sh))}
    jobs = {r: [(s, *dist.subset(c["qcodes"], c["qoff"], qs)) for s, qs in dist.local_blocks(plan, r)] for r in range(k)}
    outs = {(r, s): torch.empty((len(qo) - 1, len(sh[s])), dtype=torch.int32, device="cuda")
            for r in range(k) for s, qc, qo in jobs[r]}
    for rep in range(2):
        times, per = [], []
        for r in range(k):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            for s, qc, qo in jobs[r]:
                h.search(qc, qo, dbs[s], sw.blosum62(), 10, 2, out=outs[(r, s)])
            e1.record()
            torch.cuda.synchronize()
            times.append(e0.elapsed_time(e1) / 1e3)
print(json.dumps({"k": k, "shards": S, "tasks": mode, "opts": os.environ.get("SWDUAL_OPTS", ""), "model_s": plan.makespan,
                  "measured_max_s": max(times), "measured_sum_s": sum(times),
                  "eff_GCUPS_sum": float(ql.sum()) * float(c["doff"][-1]) / sum(times) / 1e9,
                  "searches": sum(len(jobs[r]) for r in range(k))}), flush=True)
