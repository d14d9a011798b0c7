"""swgen -- seeded synthetic protein workloads (inputs only; no SW arithmetic).

Shared by tests (oracle and GPU sides) and bench.py.  Imports neither the
oracle nor the product package.  The recipe:

* residues i.i.d. over the 20 standard amino acids at Swiss-Prot background
  composition (codes 0..19 in NCBI order ARNDCQEGHILKMFPSTWYV);
* DB lengths: lognormal body (median ~270, sigma 0.70) + 0.15 % Pareto tail
  (x_min 3000, alpha 1.6), clipped to [4, 35213] -- the paper's shortest and
  longest UniProt sequences;
* queries: the 20 standard benchmark lengths 144..5478 (sum 41,752);
* planted homologs: per query a few mutants (substitutions + short indels) at
  seeded DB positions, so scores have a realistic high tail;
* counter-based: every draw is hash(seed, stream, id, pos), so any sequence can
  be regenerated alone.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "swgen.c")
_SO = os.path.join(_HERE, "_build", "libswgen.so")
_lib = None

AMINO = "ARNDCQEGHILKMFPSTWYV"
SWEEP = [144, 189, 222, 375, 464, 567, 657, 729, 850, 1000,
         1500, 2005, 2504, 3005, 3564, 4061, 4548, 4743, 5147, 5478]

# lognormal location giving a ~360 aa mean with the tail (205M residues / 570k seqs)
MU_SWISSPROT = 5.615
SIGMA_SWISSPROT = 0.70
TAIL_FRAC = 0.0015
LMIN, LMAX = 4, 35213


def build() -> str:
    os.makedirs(os.path.dirname(_SO), exist_ok=True)
    if (not os.path.exists(_SO)) or os.path.getmtime(_SO) < os.path.getmtime(_SRC):
        tmp = _SO + ".%d.tmp" % os.getpid()
        subprocess.check_call(["gcc", "-O2", "-std=c99", "-fopenmp", "-shared", "-fPIC",
                               "-o", tmp, _SRC, "-lm"])
        os.replace(tmp, _SO)
    return _SO


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        V, I64, I32, U64, D = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int32, ctypes.c_uint64, ctypes.c_double
        lib.swgen_db_length.restype = I64
        lib.swgen_db_length.argtypes = [U64, I64, I32, D, D, D, I64, I64]
        lib.swgen_db_lengths.restype = None
        lib.swgen_db_lengths.argtypes = [U64, I64, I32, D, D, D, I64, I64, V]
        lib.swgen_db_fill.restype = None
        lib.swgen_db_fill.argtypes = [U64, I64, V, V, V]
        lib.swgen_query_fill.restype = None
        lib.swgen_query_fill.argtypes = [U64, I64, V, V]
        lib.swgen_mutate.restype = I64
        lib.swgen_mutate.argtypes = [U64, U64, V, I64, D, D, V, I64]
        _lib = lib
    return _lib


def _p(a):
    return None if a is None else a.ctypes.data_as(ctypes.c_void_p)


def make_queries(seed: int, lengths) -> tuple[np.ndarray, np.ndarray]:
    """Queries of the given lengths: (codes uint8, offsets int64[nq+1])."""
    lens = np.asarray(lengths, dtype=np.int64)
    off = np.zeros(len(lens) + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    codes = np.zeros(int(off[-1]), dtype=np.uint8)
    if len(lens):
        _load().swgen_query_fill(seed, len(lens), _p(off), _p(codes))
    return codes, off


def plan_plants(seed: int, n_db: int, n_queries: int, identities) -> list[tuple[int, int, float, int]]:
    """(db_id, query_index, identity, key) for each planted homolog; seeded, distinct ids."""
    if n_db == 0 or n_queries == 0 or not identities:
        return []
    rng = np.random.default_rng([seed, 0x504C414E54])
    total = n_queries * len(identities)
    ids = rng.choice(n_db, size=min(total, n_db), replace=False)
    out = []
    k = 0
    for qi in range(n_queries):
        for ident in identities:
            if k >= len(ids):
                break
            out.append((int(ids[k]), qi, float(ident), (seed << 32) + k))
            k += 1
    return out


def make_db(seed: int, n: int, kind: int = 0, mu: float = MU_SWISSPROT, sigma: float = SIGMA_SWISSPROT,
            tail_frac: float = TAIL_FRAC, lmin: int = LMIN, lmax: int = LMAX,
            plants=None, qcodes=None, qoff=None) -> tuple[np.ndarray, np.ndarray]:
    """Database of n sequences: (codes uint8, offsets int64[n+1]).

    kind 0 = Swiss-Prot-like lengths, kind 1 = long-tail only (> 3000 aa).
    plants = plan_plants(...) output; mutants of queries (qcodes, qoff).
    """
    lib = _load()
    lens = np.zeros(n, dtype=np.int64)
    if n:
        lib.swgen_db_lengths(seed, n, kind, mu, sigma, tail_frac, lmin, lmax, _p(lens))
    src = np.full(n, -1, dtype=np.int32)
    plants = plants or []
    for db_id, qi, ident, key in plants:
        q = np.ascontiguousarray(qcodes[qoff[qi]:qoff[qi + 1]])
        p_sub, p_indel = (1.0 - ident), (1.0 - ident) * 0.25
        lens[db_id] = max(1, lib.swgen_mutate(seed, key, _p(q), len(q), p_sub, p_indel, None, 0))
        src[db_id] = qi
    off = np.zeros(n + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    codes = np.zeros(int(off[-1]), dtype=np.uint8)
    if n:
        lib.swgen_db_fill(seed, n, _p(off), _p(src), _p(codes))
    for db_id, qi, ident, key in plants:
        q = np.ascontiguousarray(qcodes[qoff[qi]:qoff[qi + 1]])
        p_sub, p_indel = (1.0 - ident), (1.0 - ident) * 0.25
        dst = codes[off[db_id]:off[db_id + 1]]
        got = lib.swgen_mutate(seed, key, _p(q), len(q), p_sub, p_indel, _p(dst), len(dst))
        if got == 0:                      # an empty mutant keeps one residue
            dst[:] = q[:1] if len(q) else 0
    return codes, off


# BASELINE.json configs
CONFIGS = {
    "c1": dict(db_seed=1, n_db=1000, kind=0, q_seed=1, q_lens=[144], plant_ids=[1.0, 0.9, 0.75]),
    "c2": dict(db_seed=2, n_db=570_000, kind=0, q_seed=2, q_lens=[567], plant_ids=[1.0, 0.9, 0.8, 0.7]),
    "c3": dict(db_seed=2, n_db=570_000, kind=0, q_seed=3, q_lens=SWEEP, plant_ids=[1.0, 0.9, 0.8, 0.7]),
    "c4": dict(db_seed=4, n_db=1500, kind=1, q_seed=4, q_lens=[2000, 5000, 10000, 20000, 35000],
               plant_ids=[1.0, 0.95, 0.9]),
    "c5": dict(db_seed=5, n_db=50_000_000, kind=0, mu=5.545, q_seed=3, q_lens=SWEEP,
               plant_ids=[1.0, 0.9, 0.8, 0.7]),
    # PAPER.md Table V (L757-782, sec. V.C): 40-query sets vs a Swiss-Prot-sized DB.
    # Homogeneous: sizes 4,500..5,000 ("range in size from 4500 to 5000", L762-763);
    # heterogeneous: sizes 4..35,213 ("between 4 ... and 35213", L763-764).  Lengths
    # evenly spaced over each range (sum 190k / 704k; the paper's own cells, App. D,
    # imply sums of ~190k and ~700k against its 190.7M-residue UniProt).
    "t5hom": dict(db_seed=2, n_db=570_000, kind=0, q_seed=6,
                  q_lens=[4500 + (500 * i) // 39 for i in range(40)], plant_ids=[1.0, 0.8]),
    "t5het": dict(db_seed=2, n_db=570_000, kind=0, q_seed=7,
                  q_lens=[4 + ((35213 - 4) * i) // 39 for i in range(40)], plant_ids=[1.0, 0.8]),
}


def make_config(name: str, n_db: int | None = None, q_lens=None):
    """Build a named workload; n_db / q_lens override the sizes (same recipe)."""
    c = dict(CONFIGS[name])
    if n_db is not None:
        c["n_db"] = n_db
    if q_lens is not None:
        c["q_lens"] = list(q_lens)
    qcodes, qoff = make_queries(c["q_seed"], c["q_lens"])
    plants = plan_plants(c["db_seed"], c["n_db"], len(c["q_lens"]), c["plant_ids"])
    dcodes, doff = make_db(c["db_seed"], c["n_db"], kind=c["kind"], mu=c.get("mu", MU_SWISSPROT),
                           plants=plants, qcodes=qcodes, qoff=qoff)
    return dict(name=name, qcodes=qcodes, qoff=qoff, dcodes=dcodes, doff=doff, plants=plants,
                gap_open=10, gap_extend=2)


def random_seqs(rng: np.random.Generator, n: int, lmin: int, lmax: int, alpha: int = 20):
    """Small uniform random sequences for edge-case tests: (codes, offsets)."""
    lens = rng.integers(lmin, lmax + 1, size=n).astype(np.int64)
    off = np.zeros(n + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    codes = rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8)
    return codes, off


def subset(codes, off, ids):
    """Sequences `ids` (in that order) of a (codes, offsets) set: (codes, offsets)."""
    ids = np.asarray(ids, dtype=np.int64)
    lens = off[ids + 1] - off[ids]
    so = np.zeros(len(ids) + 1, dtype=np.int64)
    np.cumsum(lens, out=so[1:])
    sc = np.empty(int(so[-1]), dtype=np.uint8)
    for k, i in enumerate(ids):
        sc[so[k]:so[k + 1]] = codes[off[i]:off[i + 1]]
    return sc, so


def c5_sample(doff, n_queries: int, per_stratum: int = 625, seed: int = 0xC5):
    """SURVEY.md 8(d) C5 sampling plan (input selection only, no SW arithmetic).

    Strata = query x DB-length decile x DB-index octile (the 8 contiguous index
    ranges stand for the 8 shards of the input order): 20 x 10 x 8 = 1,600
    strata of `per_stratum` distinct sequences each (10^6 pairs at the defaults).
    Returns dict(q, d, stratum) int64 arrays sorted by (stratum, d), and cells.
    """
    doff = np.asarray(doff, dtype=np.int64)
    nd = len(doff) - 1
    lens = np.diff(doff)
    edges = np.quantile(lens, np.linspace(0, 1, 11)[1:-1], method="lower")
    dec = np.searchsorted(edges, lens, side="right")               # 0..9
    octl = (np.arange(nd, dtype=np.int64) * 8) // max(nd, 1)        # 0..7
    key = dec * 8 + octl
    order = np.argsort(key, kind="stable")
    bounds = np.searchsorted(key[order], np.arange(81))
    qs, ds, ss = [], [], []
    for qi in range(n_queries):
        for k in range(80):
            pool = order[bounds[k]:bounds[k + 1]]
            if not len(pool):
                continue
            rng = np.random.default_rng([seed, qi, k])
            pick = np.sort(rng.choice(pool, size=min(per_stratum, len(pool)), replace=False))
            qs.append(np.full(len(pick), qi, dtype=np.int64))
            ds.append(pick.astype(np.int64))
            ss.append(np.full(len(pick), qi * 80 + k, dtype=np.int64))
    q = np.concatenate(qs) if qs else np.zeros(0, np.int64)
    d = np.concatenate(ds) if ds else np.zeros(0, np.int64)
    s = np.concatenate(ss) if ss else np.zeros(0, np.int64)
    return dict(q=q, d=d, stratum=s, cells=0.0)
