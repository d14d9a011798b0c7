"""sw_align throughput on top hits: search a workload, take the
top-K hits per query, align them on the GPU (timed), and check a sample of the
alignments against the oracle.  Prints one JSON line."""
import json
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402  (test infrastructure: the sampled check only)
import swgen  # noqa: E402
from oracle.blosum62 import blosum62 as oracle_b62  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402

wl = os.environ.get("ALIGN_WORKLOAD", "c3")
top = int(os.environ.get("ALIGN_TOP", "10"))
c = swgen.make_config(wl)
h = sw.Handle(0)
db = h.load_db(c["dcodes"], c["doff"])
S = sw.blosum62()
scores = h.search(c["qcodes"], c["qoff"], db, S, 10, 2)
torch.cuda.synchronize()
sc = scores.cpu().numpy()
nq = sc.shape[0]
pairs = []
for q in range(nq):
    for d in np.argsort(-sc[q], kind="stable")[:top]:
        pairs.append((q, int(d)))
pairs = np.array(pairs, dtype=np.int32)
qlen = np.diff(c["qoff"])
dlen = np.diff(c["doff"])
cells = float(sum(qlen[q] * dlen[d] for q, d in pairs))
h.align(c["qcodes"], c["qoff"], db, pairs[:4], S, 10, 2)  # warm-up
t0 = time.perf_counter()
got = h.align(c["qcodes"], c["qoff"], db, pairs, S, 10, 2)
dt = time.perf_counter() - t0
assert all(g[0] == sc[q, d] for g, (q, d) in zip(got, pairs))
rng = np.random.default_rng(1)
sample = rng.choice(len(pairs), size=min(12, len(pairs)), replace=False)
ok = True
for k in sample:
    q, d = pairs[k]
    ref = oracle.gotoh_align(c["qcodes"][c["qoff"][q]:c["qoff"][q + 1]], c["dcodes"][c["doff"][d]:c["doff"][d + 1]],
                             oracle_b62(), 10, 2)
    ok &= tuple(got[k][:5]) == ref[:5] and got[k][5] == ref[5]
print(json.dumps({"workload": wl, "top": top, "pairs": len(pairs), "cells": cells, "align_s": round(dt, 4),
                  "GCUPS_incl_traceback_and_host_copies": round(cells / dt / 1e9, 1),
                  "mean_path_ops": float(np.mean([len(g[5]) for g in got])), "oracle_sample": int(len(sample)),
                  "oracle_sample_ok": bool(ok)}))
