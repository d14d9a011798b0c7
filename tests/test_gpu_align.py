"""GPU parity of sw_align (end cell, start cell and path of the
best local alignment) against the oracle's gotoh_align, element by element:
score, the four coordinates and every run-length operation must be identical
(the tie-breaks are DESIGN.md reading R-13, implemented independently on both
sides).  Small alphabets and random asymmetric matrices make ties frequent;
query lengths cross the kernel's 256-row strips and 2,048-row warp rounds;
DB sequences sit in both halves of the packed pairs.
"""
import ctypes

import numpy as np
import pytest

import oracle
import swgen
from oracle.blosum62 import blosum62 as oracle_b62

pytestmark = pytest.mark.gpu


def _pkg():
    import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
    return sw


def _seqs(lengths, rng, alpha):
    lens = np.asarray(lengths, dtype=np.int64)
    off = np.zeros(len(lens) + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    return rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8), off


def _run(qc, qo, dc, do, pairs, S, gs, ge, alpha, opts=None):
    sw = _pkg()
    with sw.Handle(0) as h:
        for k, v in (opts or {}).items():
            h.set_option(k, v)
        db = h.load_db(dc, do, alphabet_size=alpha)
        return h.align(qc, qo, db, pairs, S, gs, ge)


def _check(qc, qo, dc, do, pairs, S, gs, ge, alpha, opts=None):
    got = _run(qc, qo, dc, do, pairs, S.astype(np.int8), gs, ge, alpha, opts)
    for k, (q, d) in enumerate(pairs):
        ref = oracle.gotoh_align(qc[qo[q]:qo[q + 1]], dc[do[d]:do[d + 1]], S.astype(np.int32), gs, ge)
        assert got[k][:5] == ref[:5], (k, q, d, got[k][:5], ref[:5])
        assert got[k][5] == ref[5], (k, q, d, "path differs")


@pytest.mark.parametrize("alpha,gs,ge", [(4, 3, 1), (4, 0, 2), (3, 0, 0), (6, 5, 1)])
def test_align_random_ties(alpha, gs, ge):
    rng = np.random.default_rng(100 + 7 * alpha + gs + 3 * ge)
    S = rng.integers(-4, 6, size=(alpha, alpha))
    ql = [1, 2, 7, 31, 255, 256, 257, 600]
    dl = [1, 3, 4, 5, 9, 64, 250, 333, 700, 2]
    qc, qo = _seqs(ql, rng, alpha)
    dc, do = _seqs(dl, rng, alpha)
    pairs = [(q, d) for q in range(len(ql)) for d in range(len(dl))]
    _check(qc, qo, dc, do, pairs, S, gs, ge, alpha)


def test_align_multi_round_strips():
    """Queries of 2,048+ rows use every warp of the CTA and wrap round-robin."""
    rng = np.random.default_rng(5)
    alpha = 20
    S = oracle_b62()
    ql = [2047, 2048, 2049, 4700]
    dl = [300, 1201, 64, 5]
    qc, qo = _seqs(ql, rng, alpha)
    dc, do = _seqs(dl, rng, alpha)
    # plant a mutated copy of a query slice into DB sequence 1 so the path is long
    src = qc[qo[3] + 1000:qo[3] + 1000 + dl[1]].copy()
    mut = rng.random(len(src)) < 0.15
    src[mut] = rng.integers(0, alpha, size=int(mut.sum()))
    dc[do[1]:do[2]] = src
    pairs = [(q, d) for q in range(len(ql)) for d in range(len(dl))]
    _check(qc, qo, dc, do, pairs, S, 10, 2, 24)


def test_align_planted_homologs_blosum62():
    c = swgen.make_config("c1", n_db=400)
    S = oracle_b62()
    pl = [p[0] for p in c["plants"]]
    rng = np.random.default_rng(9)
    ds = sorted(set(pl) | set(rng.choice(len(c["doff"]) - 1, size=30, replace=False).tolist()))
    pairs = [(0, d) for d in ds]
    _check(c["qcodes"], c["qoff"], c["dcodes"], c["doff"], pairs, S, 10, 2, 24)


def test_align_scores_match_search_and_small_workspace():
    """Scores equal sw_search's; a tiny workspace forces one pair per batch."""
    rng = np.random.default_rng(77)
    alpha = 24
    ql = [150, 900]
    dl = list(rng.integers(1, 500, size=61)) + [0, 3000]
    qc, qo = _seqs(ql, rng, 20)
    dc, do = _seqs(dl, rng, 20)
    sw = _pkg()
    pairs = [(q, d) for q in range(2) for d in range(len(dl))]
    with sw.Handle(0) as h:
        h.set_option("align_workspace_mb", 1)
        db = h.load_db(dc, do, alphabet_size=alpha)
        out = np.zeros((2, len(dl)), dtype=np.int32)
        h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
        got = h.align(qc, qo, db, pairs, sw.blosum62(), 10, 2)
    for k, (q, d) in enumerate(pairs):
        assert got[k][0] == out[q, d]
    sample = pairs[::7] + [(1, len(dl) - 1), (0, len(dl) - 2)]
    _check(qc, qo, dc, do, sample, oracle_b62(), 10, 2, alpha)


def test_align_edges_and_errors():
    sw = _pkg()
    rng = np.random.default_rng(3)
    alpha = 4
    S = -np.ones((alpha, alpha), dtype=np.int8)  # every alignment scores < 0 -> score 0, no path
    qc, qo = _seqs([5, 0], rng, alpha)
    dc, do = _seqs([4, 0, 6], rng, alpha)
    with sw.Handle(0) as h:
        db = h.load_db(dc, do, alphabet_size=alpha)
        got = h.align(qc, qo, db, [(0, 0), (0, 1), (1, 2), (0, 2)], S, 1, 1)
        for g in got:
            assert g == (0, -1, -1, -1, -1, [])
        assert h.align(qc, qo, db, np.zeros((0, 2), dtype=np.int32), S, 1, 1) == []
        with pytest.raises(sw.SWError):
            h.align(qc, qo, db, [(0, 3)], S, 1, 1)
        with pytest.raises(sw.SWError):
            h.align(qc, qo, db, [(2, 0)], S, 1, 1)
        # an ops region too small for the path is reported, not overrun
        S2 = np.eye(alpha, dtype=np.int8) * 5 - 1
        q = np.array([0, 1, 2, 3, 0, 1], dtype=np.uint8)
        qo2 = np.array([0, 6], dtype=np.int64)
        d = np.array([0, 1, 3, 2, 3, 0, 1], dtype=np.uint8)
        db2 = h.load_db(d, np.array([0, 7], dtype=np.int64), alphabet_size=alpha)
        L = sw._lib.lib()
        pairs = np.array([[0, 0]], dtype=np.int32)
        out5 = np.zeros(5, dtype=np.int32)
        ops = np.zeros(1, dtype=np.uint32)
        offs = np.array([0, 1], dtype=np.int64)
        nops = np.zeros(1, dtype=np.int32)
        vp = lambda a: a.ctypes.data_as(ctypes.c_void_p)
        rc = L.sw_align(h.ptr, vp(q), vp(qo2), 1, db2.ptr, vp(pairs), 1, vp(S2), 0, 1, vp(out5), vp(ops),
                        vp(offs), vp(nops), None)
        ref = oracle.gotoh_align(q, d, S2.astype(np.int32), 0, 1)
        assert len(ref[5]) > 1 and rc == sw._lib.SW_EINVAL


def test_align_nucleotides_fig1_and_random():
    """Nucleotide mode (alphabet 5, ma/mi, Gs = 0 linear gap of Eq. (1)): the
    Fig. 1 pair and random DNA with many ties."""
    sw = _pkg()
    rng = np.random.default_rng(21)
    S = sw.nucleotide_matrix(1, -1)
    qs = [sw.encode_nucleotide("ACTTGTCCG"), rng.integers(0, 4, size=300).astype(np.uint8),
          rng.integers(0, 5, size=1100).astype(np.uint8)]
    qo = np.zeros(len(qs) + 1, dtype=np.int64)
    np.cumsum([len(x) for x in qs], out=qo[1:])
    qc = np.concatenate(qs)
    dl = [8, 250, 901, 33, 1]
    dc, do = _seqs(dl, rng, 4)
    dc[:8] = sw.encode_nucleotide("ATTGTCAG")
    pairs = [(q, d) for q in range(len(qs)) for d in range(len(dl))]
    for gs, ge in ((0, 2), (3, 1)):
        _check(qc, qo, dc, do, pairs, S.astype(np.int32), gs, ge, 5)
    got = _run(qc, qo, dc, do, [(0, 0)], S, 0, 2, 5)
    assert got[0][0] == 5


def test_align_very_tall_query_split_over_ctas():
    """Queries above 48 strips (12,288 rows) are split over K = strips / 8 CTAs
    chained through global rows; the K partial end cells merge in (value, j, i)
    order.  A small alphabet makes equal maxima in different CTAs likely."""
    rng = np.random.default_rng(31)
    alpha = 4
    S = rng.integers(-3, 4, size=(alpha, alpha))
    ql = [12289, 13000]
    dl = [180, 7, 640]
    qc, qo = _seqs(ql, rng, alpha)
    dc, do = _seqs(dl, rng, alpha)
    dc[do[2]:do[2] + 500] = qc[qo[1] + 9000:qo[1] + 9500]   # a long diagonal in the lower CTAs
    pairs = [(q, d) for q in range(len(ql)) for d in range(len(dl))]
    _check(qc, qo, dc, do, pairs, S, 2, 1, alpha)
