"""Probe: time of single long work items in the intra-task (chained-warp) mode.
One query of length M against K sequences of length L (all long pairs).
Prints JSON per case.  Not part of the product path."""
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402

cases = [(35000, 2, 35213), (35000, 600, 35213), (5000, 2, 35213), (35000, 2, 4000), (20000, 600, 7000),
         (4096, 2, 35213), (512, 2, 35213), (512, 592, 35213), (1024, 2, 35213), (8192, 2, 35213)]
rng = np.random.default_rng(1)
h = sw.Handle(0, timing=True)
h.set_option("t_long", 64)
for M, K, L in cases:
    dc, do = swgen.random_seqs(rng, K, L, L)
    qc, qo = swgen.random_seqs(rng, 1, M, M)
    db = h.load_db(dc, do)
    out = torch.empty((1, K), dtype=torch.int32, device="cuda")
    h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1)
    cells = float(M) * K * L
    strips = (M + 511) // 512
    print(json.dumps({"M": M, "K": K, "L": L, "strips": strips, "ms": round(ms, 3),
                      "ns_per_step_if_8_warps": round(ms * 1e6 / (((strips + 7) // 8) * (L + 64) + min(strips, 8) * 96), 1),
                      "GCUPS": round(cells / ms / 1e6, 1),
                      "per_item_GCUPS": round(cells / min(K // 2 or 1, 296) / ms / 1e6, 2)}), flush=True)
    db.free()
