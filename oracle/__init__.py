"""oracle/ -- TEST INFRASTRUCTURE ONLY.

A plain, single-threaded CPU implementation of what the SWDUAL hot path
computes: many-query x database Smith-Waterman/Gotoh local-alignment scores
(Eqs. (2)-(4) L170-194).  See sw_oracle.c for the
line-by-line citation of each step.

Only tests/, __graft_entry__.smoke() and bench.py (cpu_baseline leg and
``--impl reference``) may import this package.  The product package
(paper_conf_icpp_kedad_sidhoummmmt14_b200) never imports it and shares no code
with it.  Pins: tests/test_oracle_pins.py (brute force, textbook values,
special cases, invariants, worked goldens under tests/golden/).

Parity status: oracle_gotoh_score / gotoh_search / gotoh_align are pinned (see
DESIGN.md "Oracle pins"); nothing here is "parity unpinned".
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from concurrent.futures import ThreadPoolExecutor

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "sw_oracle.c")
_SO = os.path.join(_HERE, "_build", "libsworacle.so")
_lib = None


def build() -> str:
    """Compile sw_oracle.c with plain gcc (no SIMD intrinsics in the source)."""
    os.makedirs(os.path.dirname(_SO), exist_ok=True)
    if (not os.path.exists(_SO)) or os.path.getmtime(_SO) < os.path.getmtime(_SRC):
        tmp = _SO + ".%d.tmp" % os.getpid()
        subprocess.check_call(["gcc", "-O2", "-std=c99", "-shared", "-fPIC", "-o", tmp, _SRC])
        os.replace(tmp, _SO)
    return _SO


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        lib.oracle_gotoh_score.restype = ctypes.c_int32
        lib.oracle_gotoh_score.argtypes = [
            ctypes.c_void_p, ctypes.c_int64, ctypes.c_void_p, ctypes.c_int64,
            ctypes.c_void_p, ctypes.c_int32, ctypes.c_int32, ctypes.c_int32]
        lib.oracle_gotoh_search.restype = ctypes.c_int32
        lib.oracle_gotoh_search.argtypes = [
            ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int64,
            ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int64,
            ctypes.c_int64, ctypes.c_int64,
            ctypes.c_void_p, ctypes.c_int32, ctypes.c_int32, ctypes.c_int32,
            ctypes.c_void_p]
        lib.oracle_gotoh_align.restype = ctypes.c_int32
        lib.oracle_gotoh_align.argtypes = [
            ctypes.c_void_p, ctypes.c_int64, ctypes.c_void_p, ctypes.c_int64,
            ctypes.c_void_p, ctypes.c_int32, ctypes.c_int32, ctypes.c_int32,
            ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int32]
        _lib = lib
    return _lib


def _ptr(a: np.ndarray):
    return a.ctypes.data_as(ctypes.c_void_p)


def _matrix(S) -> np.ndarray:
    S = np.ascontiguousarray(np.asarray(S, dtype=np.int32))
    assert S.ndim == 2 and S.shape[0] == S.shape[1]
    return S


def gotoh_score(q, d, S, gs: int, ge: int) -> int:
    """Score of one (query, subject) pair; q, d are uint8 code arrays."""
    q = np.ascontiguousarray(np.asarray(q, dtype=np.uint8))
    d = np.ascontiguousarray(np.asarray(d, dtype=np.uint8))
    S = _matrix(S)
    v = _load().oracle_gotoh_score(_ptr(q), len(q), _ptr(d), len(d), _ptr(S), S.shape[0], int(gs), int(ge))
    if v < 0:
        raise ValueError("oracle: bad input (code >= alphabet size or OOM)")
    return int(v)


def _search_chunk(args):
    qcodes, qoff, dcodes, doff, b0, b1, S, gs, ge = args
    nq = len(qoff) - 1
    sub = np.ascontiguousarray(doff[b0:b1 + 1])          # offsets stay absolute into dcodes
    out = np.zeros((nq, b1 - b0), dtype=np.int32)
    rc = _load().oracle_gotoh_search(_ptr(qcodes), _ptr(qoff), nq, _ptr(dcodes), _ptr(sub), b1 - b0,
                                     0, b1 - b0, _ptr(S), S.shape[0], int(gs), int(ge), _ptr(out))
    if rc != 0:
        raise ValueError("oracle: bad input")
    return b0, b1, out


def gotoh_search(qcodes, qoff, dcodes, doff, S, gs: int, ge: int, procs: int = 1) -> np.ndarray:
    """scores[q][d] for every query x database pair (L196-201).

    procs > 1 splits the database into disjoint subsets scored by independent
    worker threads (each runs the same plain, single-threaded C loop; ctypes
    releases the GIL for the call).  Threads, not forked processes: forking a
    process that already runs CUDA / torch threads can deadlock the child.
    """
    qcodes = np.ascontiguousarray(qcodes, dtype=np.uint8)
    dcodes = np.ascontiguousarray(dcodes, dtype=np.uint8)
    qoff = np.ascontiguousarray(qoff, dtype=np.int64)
    doff = np.ascontiguousarray(doff, dtype=np.int64)
    S = _matrix(S)
    nq, nd = len(qoff) - 1, len(doff) - 1
    if nq == 0 or nd == 0:
        return np.zeros((nq, nd), dtype=np.int32)
    if procs <= 1:
        return _search_chunk((qcodes, qoff, dcodes, doff, 0, nd, S, gs, ge))[2]
    # balance by residues
    cum = doff[1:] - doff[0]
    tot = int(cum[-1]) if nd else 0
    nchunks = procs * 4
    cuts = [0] + [int(np.searchsorted(cum, tot * k / nchunks)) for k in range(1, nchunks)] + [nd]
    cuts = sorted(set(cuts))
    jobs = [(qcodes, qoff, dcodes, doff, a, b, S, gs, ge) for a, b in zip(cuts[:-1], cuts[1:]) if b > a]
    out = np.zeros((nq, nd), dtype=np.int32)
    build()
    with ThreadPoolExecutor(max_workers=procs) as pool:
        for b0, b1, blk in pool.map(_search_chunk, jobs):
            out[:, b0:b1] = blk
    return out


def gotoh_align(q, d, S, gs: int, ge: int):
    """Best local alignment of one pair (sw_oracle.c oracle_gotoh_align):
    (score, q_begin, q_end, d_begin, d_end, ops) with ops run-length codes
    (len << 2 | op), op 0 = M, 1 = I (query vs gap), 2 = D (subject vs gap)."""
    q = np.ascontiguousarray(np.asarray(q, dtype=np.uint8))
    d = np.ascontiguousarray(np.asarray(d, dtype=np.uint8))
    S = _matrix(S)
    out5 = np.zeros(5, dtype=np.int32)
    ops = np.zeros(len(q) + len(d) + 1, dtype=np.uint32)
    n = _load().oracle_gotoh_align(_ptr(q), len(q), _ptr(d), len(d), _ptr(S), S.shape[0], int(gs), int(ge),
                                   _ptr(out5), _ptr(ops), len(ops))
    if n < 0:
        raise ValueError("oracle: bad input (code >= alphabet size or OOM)")
    return (int(out5[0]), int(out5[1]), int(out5[2]), int(out5[3]), int(out5[4]), [int(x) for x in ops[:n]])
