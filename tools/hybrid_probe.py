"""Hybrid SWDUAL on one B200 box: GPU-only vs GPU + host-core
PEs placed by the dual approximation, same workload, wall time of the whole
search (host output).  Rates are calibrated first on the same box."""
import json
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402
from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist  # noqa: E402

wl = os.environ.get("HYB_WORKLOAD", "c3")
n_shards = int(os.environ.get("HYB_SHARDS", "32"))
cores = os.cpu_count() or 1
n_cpus = int(os.environ.get("HYB_CPUS", str(max(1, cores - 2))))
c = swgen.make_config(wl)
S = sw.blosum62()
h = sw.Handle(0)
hdb = dist.HybridDB(h, c["dcodes"], c["doff"], n_shards=n_shards)
qlen = np.diff(c["qoff"])
cells = float(qlen.sum()) * float(c["doff"][-1] - c["doff"][0])
# calibrate: GPU rate from one full GPU-only search, CPU rate from one PE on a slice
plan0 = hdb.plan(qlen, 0, 1.0, 1.0)
hdb.search(c["qcodes"], c["qoff"], S, plan=plan0)
t = time.perf_counter(); ref, _ = hdb.search(c["qcodes"], c["qoff"], S, plan=plan0); t_gpu = time.perf_counter() - t
gpu_rate = cells / t_gpu
# per-query GPU rates (the GPU's cell rate depends on the query length)
db_full = h.load_db(c["dcodes"], c["doff"])
rates = []
for q in range(len(qlen)):
    qq, oo = c["qcodes"][c["qoff"][q]:c["qoff"][q + 1]], np.array([0, qlen[q]], dtype=np.int64)
    out = torch.empty((1, db_full.n_seqs), dtype=torch.int32, device="cuda")
    h.search(qq, oo, db_full, S, 10, 2, out=out)
    torch.cuda.synchronize()
    t = time.perf_counter()
    h.search(qq, oo, db_full, S, 10, 2, out=out)
    torch.cuda.synchronize()
    rates.append(float(qlen[q]) * float(c["doff"][-1] - c["doff"][0]) / (time.perf_counter() - t))
db_full.free()
gpu_rate_q = np.array(rates) * (gpu_rate / (cells / sum(float(qlen[q]) * float(c["doff"][-1] - c["doff"][0]) / rates[q] for q in range(len(qlen)))))
sl = hdb.host[0]
k = min(len(sl[1]) - 1, 3000)
qc, qo = swgen.make_queries(5, [567])
t = time.perf_counter()
sw.search_cpu(qc, qo, sl[0][:sl[1][k] - sl[1][0]], sl[1][:k + 1] - sl[1][0], S, 10, 2, n_threads=1)
cpu_rate = 567.0 * float(sl[1][k] - sl[1][0]) / (time.perf_counter() - t)
plan = hdb.plan(qlen, n_cpus, gpu_rate_q, cpu_rate)
hdb.search(c["qcodes"], c["qoff"], S, plan=plan)
t = time.perf_counter(); got, info = hdb.search(c["qcodes"], c["qoff"], S, plan=plan); t_hyb = time.perf_counter() - t
cpu_cells = sum(float(qlen[q]) * hdb.residues[s] for (q, s), p in zip(plan.tasks, plan.pe) if p < n_cpus)
print(json.dumps({"workload": wl, "shards": n_shards, "tasks": len(plan.tasks), "host_cores": cores, "cpu_pes": n_cpus,
                  "gpu_rate_GCUPS": round(gpu_rate / 1e9, 1), "gpu_rate_per_query_GCUPS": [round(r / 1e9) for r in gpu_rate_q], "cpu_pe_rate_GCUPS": round(cpu_rate / 1e9, 2),
                  "gpu_only_s": round(t_gpu, 4), "hybrid_s": round(t_hyb, 4),
                  "hybrid_GCUPS": round(cells / t_hyb / 1e9, 1), "gpu_only_GCUPS": round(cells / t_gpu / 1e9, 1),
                  "tasks_on_cpus": int((plan.pe < n_cpus).sum()), "cell_share_on_cpus": round(cpu_cells / cells, 5),
                  "model_makespan_s": round(plan.makespan, 4), "lambda_s": round(plan.lam, 4),
                  "cpu_pe_busy_s_max": round(max(info["cpu_s"]) if info["cpu_s"] else 0.0, 4),
                  "identical_to_gpu_only": bool(np.array_equal(got, ref))}))
