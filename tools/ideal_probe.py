"""Probe: the scoring kernel on idealised workloads (equal DB lengths, query
lengths a multiple of the strip height) vs config-3-like ones, to split the gap
to the roofline between the inner loop and workload structure (padding, tail,
pass fill).  Not part of the product path.  Prints JSON per case."""
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402

rng = np.random.default_rng(7)
h = sw.Handle(0, timing=True)


def seqs(n, lo, hi):
    return swgen.random_seqs(rng, n, lo, hi)


cases = [
    ("eq400_q1920x20", 150_000, 400, 400, [1920] * 20),
    ("eq400_q1920x2", 150_000, 400, 400, [1920] * 2),
    ("eq400_q96x40", 300_000, 400, 400, [96] * 40),
    ("eq2000_q1920x20", 30_000, 2000, 2000, [1920] * 20),
    ("u300_500_q1920x20", 150_000, 300, 500, [1920] * 20),
    ("eq400_q2000x20", 150_000, 400, 400, [2000] * 20),
]
for name, n, lo, hi, ql in cases:
    dc, do = seqs(n, lo, hi)
    qs = [seqs(1, m, m) for m in ql]
    qc = np.concatenate([q[0] for q in qs])
    qo = np.concatenate([[0], np.cumsum(ql)]).astype(np.int64)
    db = h.load_db(dc, do)
    out = torch.empty((len(ql), n), dtype=torch.int32, device="cuda")
    for _ in range(2):
        h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
    e1.record()
    torch.cuda.synchronize()
    st = h.last_stats()
    ms = e0.elapsed_time(e1)
    print(json.dumps({"case": name, "ms": round(ms, 2), "GCUPS": round(st["cells"] / ms / 1e6, 1),
                      "kernel_GCUPS": round(st["cells"] / st["short_ms"] / 1e6, 1),
                      "computed_over_cells": round(st["cells_computed"] / st["cells"], 4),
                      "G": st.get("last_G"), "R": st.get("last_R")}), flush=True)
    db.free()
