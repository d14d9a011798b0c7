"""Probe: config-3 DB, each query pair (mode 1) alone and all together; kernel vs search time."""
import json, os, sys
import numpy as np
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402

c = swgen.make_config("c3")
h = sw.Handle(0, timing=True)
db = h.load_db(c["dcodes"], c["doff"])
N = db.n_seqs
ql = np.diff(c["qoff"])
cases = [[i, i + 1] for i in range(0, len(ql), 2)] + [list(range(len(ql)))]
for sel in cases:
    qc = np.concatenate([c["qcodes"][c["qoff"][i]:c["qoff"][i + 1]] for i in sel])
    qo = np.concatenate([[0], np.cumsum(ql[sel])]).astype(np.int64)
    out = torch.empty((len(sel), N), dtype=torch.int32, device="cuda")
    h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(); h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out); e1.record(); torch.cuda.synchronize()
    st = h.last_stats()
    ms = e0.elapsed_time(e1)
    print(json.dumps({"queries": [int(ql[i]) for i in sel], "ms": round(ms, 2), "kernel_ms": round(st["short_ms"], 2),
                      "GCUPS": round(st["cells"] / ms / 1e6, 1), "kernel_GCUPS": round(st["cells"] / st["short_ms"] / 1e6, 1),
                      "n_overflow": st["n_overflow"]}), flush=True)

# geometry sweep for two representative query pairs (mode 1)
for sel in ([4, 5], [18, 19]):
    qc = np.concatenate([c["qcodes"][c["qoff"][i]:c["qoff"][i + 1]] for i in sel])
    qo = np.concatenate([[0], np.cumsum(ql[sel])]).astype(np.int64)
    out = torch.empty((len(sel), N), dtype=torch.int32, device="cuda")
    res = []
    for G in (4, 8, 16):
        for R in (8, 12, 16, 20, 24, 28, 32):
            h.set_option("force_G", G); h.set_option("force_R", R)
            h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out); torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(); h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out); e1.record(); torch.cuda.synchronize()
            st = h.last_stats()
            res.append((round(st["cells"] / e0.elapsed_time(e1) / 1e6, 1), G, R))
    h.set_option("force_G", 0); h.set_option("force_R", 0)
    print(json.dumps({"pair": [int(ql[i]) for i in sel], "best": sorted(res, reverse=True)[:8]}), flush=True)
