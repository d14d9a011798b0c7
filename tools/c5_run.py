"""BASELINE config 5 on ONE B200: TrEMBL-scale synthetic DB (~50M sequences,
~17G residues) x the 20-query sweep, sampled parity against the CPU oracle
(seeded random sample + every planted homolog + top hits).

The north star shards C5 over 8 GPUs; this run puts all of it on one GPU (the
DB fits in 180 GB of HBM), which is the per-GPU work x 8.  Prints one JSON line.
  python tools/c5_run.py [--n-db N] [--sample K]
"""
import argparse
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
    ap = argparse.ArgumentParser()
    ap.add_argument("--n-db", type=int, default=None)
    ap.add_argument("--sample", type=int, default=2000)
    args = ap.parse_args()
    t0 = time.time()
    c = swgen.make_config("c5", n_db=args.n_db)
    t_gen = time.time() - t0
    N = len(c["doff"]) - 1
    res = int(c["doff"][-1])
    q_lens = np.diff(c["qoff"])
    h = sw.Handle(0, timing=True)
    t0 = time.time()
    db = h.load_db(c["dcodes"], c["doff"])
    t_load = time.time() - t0
    out = torch.empty((len(q_lens), N), dtype=torch.int32, device="cuda")
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    h.search(c["qcodes"], c["qoff"], db, sw.blosum62(), 10, 2, out=out)
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1)
    st = h.last_stats()
    cells = float(q_lens.sum()) * res
    got = out.cpu().numpy()
    # sampled parity
    import oracle
    from oracle.blosum62 import blosum62 as ob62
    rng = np.random.default_rng(55)
    sample = set(rng.choice(N, size=min(N, args.sample), replace=False).tolist())
    sample |= {p[0] for p in c["plants"]}
    sample |= set(np.argsort(got.max(axis=0))[-20:].tolist())
    idx = np.array(sorted(sample), dtype=np.int64)
    from paper_conf_icpp_kedad_sidhoummmmt14_b200.dist import subset
    sc, so = subset(c["dcodes"], c["doff"], idx)
    t0 = time.time()
    ref = oracle.gotoh_search(c["qcodes"], c["qoff"], sc, so, ob62(), 10, 2, procs=os.cpu_count() or 1)
    t_or = time.time() - t0
    ok = bool(np.array_equal(got[:, idx], ref))
    print(json.dumps({"workload": "c5 on 1 GPU", "n_db": N, "residues": res, "queries": int(len(q_lens)),
                      "cells": cells, "search_ms": round(ms, 1), "GCUPS": round(cells / ms / 1e6, 1),
                      "kernel_ms": round(st["short_ms"], 1), "n_overflow": st["n_overflow"],
                      "gen_s": round(t_gen, 1), "load_s": round(t_load, 1),
                      "parity_sample": int(len(idx)), "parity_ok": ok, "oracle_s": round(t_or, 1)}), flush=True)
    if not ok:
        bad = np.argwhere(got[:, idx] != ref)
        print("MISMATCH", bad[:10].tolist(), flush=True)
        sys.exit(1)


if __name__ == "__main__":
    main()
