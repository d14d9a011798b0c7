"""Tuning probe (GPU): GCUPS of the inter-task kernel per (G, R) for a few query
lengths against the Swiss-Prot-sized synthetic DB, plus the auto choice.
Prints one JSON object per line.  Not part of the product path."""
import json
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402


def main():
    n_db = int(os.environ.get("SWEEP_NDB", "570000"))
    qlens = [int(x) for x in os.environ.get("SWEEP_Q", "144,567,1500,5478").split(",")]
    geoms = os.environ.get("SWEEP_GEOMS", "auto")
    c = swgen.make_config("c2", n_db=n_db)
    h = sw.Handle(0, timing=True)
    db = h.load_db(c["dcodes"], c["doff"])
    S = sw.blosum62()
    info = db.info()
    print(json.dumps({"db": info}), flush=True)
    for m in qlens:
        qc, qo = swgen.make_queries(77, [m])
        out = torch.empty((1, info["n_seqs"]), dtype=torch.int32, device="cuda")
        cand = [(0, 0)]
        if geoms != "auto":
            cand += [(g, r) for g in (4, 8, 16, 32) for r in (8, 12, 16, 20, 24, 28, 32)]
        for G, R in cand:
            h.set_option("force_G", G)
            h.set_option("force_R", R)
            h.search(qc, qo, db, S, 10, 2, out=out)
            torch.cuda.synchronize()
            reps = 3
            ms = []
            for _ in range(reps):
                t0 = torch.cuda.Event(enable_timing=True)
                t1 = torch.cuda.Event(enable_timing=True)
                t0.record()
                h.search(qc, qo, db, S, 10, 2, out=out)
                t1.record()
                torch.cuda.synchronize()
                ms.append(t0.elapsed_time(t1))
            st = h.last_stats()
            best = min(ms)
            print(json.dumps({"m": m, "G": st["last_G"], "R": st["last_R"], "ms": round(best, 3),
                              "search_ms": round(st["search_ms"], 3), "short_ms": round(st["short_ms"], 3),
                              "long_ms": round(st["long_ms"], 3),
                              "GCUPS": round(st["cells"] / best / 1e6, 1),
                              "short_GCUPS": round(st["cells_short"] / st["short_ms"] / 1e6, 1),
                              "pad_frac": round(1 - st["cells"] / st["cells_computed"], 4)}), flush=True)
    h.close()


if __name__ == "__main__":
    main()
