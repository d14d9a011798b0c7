"""Write full-config parity goldens from the CPU ORACLE ONLY (never the CUDA path).

North star: "bit-exact int32 scores vs the CPU oracle on all five configs"
(BASELINE.json); SURVEY.md 8(c) P7 and 8(d)'s oracle plan (C2, C3, C4 full;
C5 sampled: the m = 144 query in full, >= 10^6 stratified pairs, every planted
pair).  The paper's method is exact, so the expected values
are the oracle's Gotoh scores (oracle/sw_oracle.c, Eqs. (2)-(4) L170-194).

This script imports only `oracle` (the arithmetic) and `swgen` (seeded inputs,
no SW arithmetic).  It stores, per config, under tests/golden/:

* the SHA-256 of the generated inputs (q codes, q offsets, DB codes, DB offsets,
  little-endian), so a host-dependent change of the generated workload is
  reported as such instead of as a score mismatch;
* per query: the SHA-256 of the full int32 score row (caller DB order), its
  max / argmax / sum, and 64-bit BLAKE2b hashes of consecutive blocks of
  BLOCK sequences (to localise a mismatch);
* for C5 (sample): the stratified pair sample is defined by swgen.c5_sample
  (seeded, input-only); per stratum the BLAKE2b of the oracle scores, plus the
  planted pairs' scores in clear.

Usage (CPU box, once; ~2 h on 8 cores for everything):
  python tools/make_goldens.py --configs c1,c2,c4,c3,c5 --procs 8
"""
import argparse
import hashlib
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import oracle  # noqa: E402
import swgen  # noqa: E402
from oracle.blosum62 import blosum62  # noqa: E402

BLOCK = 16384
OUT = os.path.join(ROOT, "tests", "golden")


def inputs_sha(c):
    h = hashlib.sha256()
    for k in ("qcodes", "qoff", "dcodes", "doff"):
        a = np.ascontiguousarray(c[k])
        h.update(a.astype(a.dtype.newbyteorder("<"), copy=False).tobytes())
    return h.hexdigest()


def row_record(qi, row):
    row = np.ascontiguousarray(row, dtype="<i4")
    blocks = [hashlib.blake2b(row[b:b + BLOCK].tobytes(), digest_size=8).hexdigest()
              for b in range(0, len(row), BLOCK)]
    return {"q": int(qi), "sha256": hashlib.sha256(row.tobytes()).hexdigest(),
            "max": int(row.max()) if len(row) else 0, "argmax": int(row.argmax()) if len(row) else -1,
            "sum": int(row.astype(np.int64).sum()), "blocks": blocks}


def write(name, rec):
    path = os.path.join(OUT, name)
    tmp = path + ".tmp"
    with open(tmp, "w") as f:
        json.dump(rec, f, indent=0, sort_keys=True)
        f.write("\n")
    os.replace(tmp, path)
    print("wrote", path, flush=True)


def full_config(name, procs):
    t0 = time.time()
    c = swgen.make_config(name)
    sha = inputs_sha(c)
    nq, nd = len(c["qoff"]) - 1, len(c["doff"]) - 1
    print(f"{name}: {nq} queries x {nd} seqs, generated in {time.time() - t0:.1f}s; oracle ...", flush=True)
    t1 = time.time()
    ref = oracle.gotoh_search(c["qcodes"], c["qoff"], c["dcodes"], c["doff"], blosum62(), 10, 2, procs=procs)
    dt = time.time() - t1
    cells = float(np.diff(c["qoff"]).sum()) * float(c["doff"][-1])
    write(f"full_{name}.json", {
        "config": name, "generator": "swgen.make_config(%r)" % name, "inputs_sha256": sha,
        "n_queries": nq, "n_db": nd, "residues": int(c["doff"][-1]), "cells": cells,
        "matrix": "BLOSUM62", "gap_open": 10, "gap_extend": 2, "block": BLOCK,
        "oracle_s": round(dt, 1), "oracle_procs": procs,
        "rows": [row_record(i, ref[i]) for i in range(nq)]})


_G = {}


def _rows_worker(args):
    """One slice of the DB against one query, in a forked worker: the DB arrays are
    inherited from the parent (module global), never pickled (C5's are 17 GB)."""
    qi, b0, b1 = args
    c = _G["c"]
    qc = np.ascontiguousarray(c["qcodes"][c["qoff"][qi]:c["qoff"][qi + 1]])
    qo = np.array([0, len(qc)], dtype=np.int64)
    off = c["doff"][b0:b1 + 1]
    dc = c["dcodes"][int(off[0]):int(off[-1])]
    return qi, b0, oracle.gotoh_search(qc, qo, dc, off - off[0], _G["S"], 10, 2, procs=1)[0]


def _pairs_worker(args):
    """Oracle scores of sampled (query, sequence) pairs of one query (forked worker)."""
    qi, ids = args
    c = _G["c"]
    sc, so = swgen.subset(c["dcodes"], c["doff"], ids)
    qc = np.ascontiguousarray(c["qcodes"][c["qoff"][qi]:c["qoff"][qi + 1]])
    qo = np.array([0, len(qc)], dtype=np.int64)
    return qi, ids, oracle.gotoh_search(qc, qo, sc, so, _G["S"], 10, 2, procs=1)[0]


def c5(procs, n_db=None):
    t0 = time.time()
    c = swgen.make_config("c5", n_db=n_db)
    sha = inputs_sha(c)
    nq, nd = len(c["qoff"]) - 1, len(c["doff"]) - 1
    print(f"c5: {nq} queries x {nd} seqs, {int(c['doff'][-1])} residues, generated in "
          f"{time.time() - t0:.1f}s", flush=True)
    S = blosum62()
    import multiprocessing as mp
    _G["c"], _G["S"] = c, S
    oracle.build()
    ctx = mp.get_context("fork")
    # (i) the m = 144 query (query 0) against the whole DB, in residue-balanced slices
    t1 = time.time()
    cum = c["doff"][1:] - c["doff"][0]
    nchunks = procs * 16
    cuts = sorted(set([0] + [int(np.searchsorted(cum, int(cum[-1]) * k // nchunks)) for k in range(1, nchunks)]
                      + [nd]))
    row = np.zeros(nd, dtype=np.int32)
    with ctx.Pool(procs) as pool:
        for _qi, b0, part in pool.imap_unordered(_rows_worker, [(0, a, b) for a, b in zip(cuts[:-1], cuts[1:]) if b > a]):
            row[b0:b0 + len(part)] = part
    t_row = time.time() - t1
    print(f"c5 query-0 row in {t_row:.0f}s", flush=True)
    # (ii) stratified sample, (iii) planted pairs
    smp = swgen.c5_sample(c["doff"], nq)
    t1 = time.time()
    scores = np.zeros(len(smp["q"]), dtype=np.int32)
    jobs = []
    for qi in range(nq):
        sel = np.nonzero(smp["q"] == qi)[0]
        for part in np.array_split(sel, procs):
            if len(part):
                jobs.append((qi, smp["d"][part]))
    pos = {}
    for qi in range(nq):
        sel = np.nonzero(smp["q"] == qi)[0]
        for k, d in enumerate(smp["d"][sel]):
            pos[(qi, int(d))] = int(sel[k])
    with ctx.Pool(procs) as pool:
        for qi, ids, vals in pool.imap_unordered(_pairs_worker, jobs):
            for d, v in zip(ids, vals):
                scores[pos[(qi, int(d))]] = v
    t_smp = time.time() - t1
    smp["cells"] = float((np.diff(c["qoff"])[smp["q"]] * np.diff(c["doff"])[smp["d"]]).sum())
    strata = {}
    for s in np.unique(smp["stratum"]):
        sel = np.nonzero(smp["stratum"] == s)[0]
        strata[str(int(s))] = hashlib.blake2b(np.ascontiguousarray(scores[sel], dtype="<i4").tobytes(),
                                              digest_size=8).hexdigest()
    planted = []
    for db_id, qi, ident, key in c["plants"]:
        dc = np.ascontiguousarray(c["dcodes"][c["doff"][db_id]:c["doff"][db_id + 1]])
        qc = np.ascontiguousarray(c["qcodes"][c["qoff"][qi]:c["qoff"][qi + 1]])
        planted.append({"q": int(qi), "d": int(db_id), "identity": ident,
                        "score": oracle.gotoh_score(qc, dc, S, 10, 2)})
    write("c5_sample.json" if n_db is None else f"c5_sample_n{n_db}.json", {
        "config": "c5", "generator": "swgen.make_config('c5')", "inputs_sha256": sha,
        "n_queries": nq, "n_db": nd, "residues": int(c["doff"][-1]), "matrix": "BLOSUM62",
        "gap_open": 10, "gap_extend": 2, "block": BLOCK,
        "row_q0": row_record(0, row), "row_q0_oracle_s": round(t_row, 1),
        "sample": {"recipe": "swgen.c5_sample(doff, n_queries)", "pairs": int(len(scores)),
                   "cells": float(smp["cells"]), "oracle_s": round(t_smp, 1),
                   "all_sha256": hashlib.sha256(np.ascontiguousarray(scores, dtype="<i4").tobytes()).hexdigest(),
                   "strata_blake2b": strata},
        "planted": planted, "oracle_procs": procs})


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--configs", default="c1,c2,c4,c3,c5")
    ap.add_argument("--procs", type=int, default=os.cpu_count() or 1)
    ap.add_argument("--c5-n-db", type=int, default=None, help="smaller C5 (dry run of the recipe)")
    args = ap.parse_args()
    os.makedirs(OUT, exist_ok=True)
    for name in args.configs.split(","):
        if name == "c5":
            c5(args.procs, args.c5_n_db)
        else:
            full_config(name, args.procs)


if __name__ == "__main__":
    main()
