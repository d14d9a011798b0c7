"""Pins for the CPU oracle (oracle/): each test checks it against something the
paper or mathematics fixes, NOT against a retyping of its own recurrence.

Pins:
  P1 Fig. 1 worked example            test_fig1_*
  P2 textbook SW value                                      test_textbook
  P3 exhaustive enumeration on tiny inputs                  test_brute_*
  P4 special cases: Gs=0 -> Eq. (1); huge gaps -> Kadane;   test_special_*
     single residues
  P5 invariants (non-negativity, swap symmetry, bounds,     test_invariant_*
     monotonicity, appending, PAD)
  P6 BLOSUM62 goldens with the Gs + k*Ge discriminators     test_goldens
"""
import os

import numpy as np
import pytest

import oracle
from oracle.blosum62 import blosum62, encode
from tests import brute
from tests.brute import brute_local, linear_sw, score_alignment, ungapped_best

GOLD = os.path.join(os.path.dirname(__file__), "golden")
B62 = blosum62()


def _dna_matrix(ma, mi):
    S = np.full((4, 4), mi, dtype=np.int32)
    np.fill_diagonal(S, ma)
    return S


def _dna(s):
    return np.array(["ACGT".index(c) for c in s], dtype=np.uint8)


# ---------------------------------------------------------------- P1, P2
def test_fig1_given_alignment_scores_4():
    # the printed alignment and its score
    assert score_alignment("ACTTGTCCG", "A-TTGTCAG", 1, -1, -2) == 4


def test_fig1_local_optimum():
    q, d, S = _dna("ACTTGTCCG"), _dna("ATTGTCAG"), _dna_matrix(1, -1)
    v = oracle.gotoh_score(q, d, S, 0, 2)
    assert v == brute_local(q, d, S, 0, 2) == 5
    assert v >= 4  # the local optimum is at least the printed global alignment's score


def test_textbook():
    rows = [l.rstrip("\n").split("\t") for l in open(os.path.join(GOLD, "textbook.tsv")) if not l.startswith("#")]
    assert rows
    for name, q, d, ma, mi, gs, ge, score, _src in rows:
        S = _dna_matrix(int(ma), int(mi))
        assert oracle.gotoh_score(_dna(q), _dna(d), S, int(gs), int(ge)) == int(score), name


# ---------------------------------------------------------------- P6
def test_goldens():
    rows = [l.rstrip("\n").split("\t") for l in open(os.path.join(GOLD, "blosum62_gs10_ge2.tsv"))
            if l.strip() and not l.startswith("#")]
    assert len(rows) == 15
    for q, d, score, alt, _how in rows:
        qc, dc = encode(q), encode(d)
        got = oracle.gotoh_score(qc, dc, B62, 10, 2)
        assert got == int(score), (q, d)
        assert brute_local(qc, dc, B62, 10, 2) == int(score), (q, d)
        # the rejected reading gap(k) = Gs + (k-1)*Ge == (Gs - Ge) + k*Ge
        assert oracle.gotoh_score(qc, dc, B62, 8, 2) == int(alt), (q, d)


# ---------------------------------------------------------------- P3
@pytest.mark.parametrize("seed", range(6))
def test_brute_random_asymmetric(seed):
    """Random ASYMMETRIC matrices catch transposed S operands; random gaps catch gap-cost slips."""
    rng = np.random.default_rng(seed)
    for _ in range(25):
        A = int(rng.integers(2, 6))
        S = rng.integers(-6, 8, size=(A, A)).astype(np.int32)
        m, n = int(rng.integers(1, 7)), int(rng.integers(1, 7))
        q = rng.integers(0, A, m).astype(np.uint8)
        d = rng.integers(0, A, n).astype(np.uint8)
        gs, ge = int(rng.integers(0, 6)), int(rng.integers(0, 4))
        assert oracle.gotoh_score(q, d, S, gs, ge) == brute_local(q, d, S, gs, ge), (S, q, d, gs, ge)


@pytest.mark.parametrize("seed", range(4))
def test_brute_blosum62(seed):
    rng = np.random.default_rng(100 + seed)
    for _ in range(20):
        m, n = int(rng.integers(1, 8)), int(rng.integers(1, 8))
        q = rng.integers(0, 20, m).astype(np.uint8)
        d = rng.integers(0, 20, n).astype(np.uint8)
        for gs, ge in ((10, 2), (0, 1), (3, 1), (11, 1)):
            assert oracle.gotoh_score(q, d, B62, gs, ge) == brute_local(q, d, B62, gs, ge)


# ---------------------------------------------------------------- P4
@pytest.mark.parametrize("seed", range(4))
def test_special_gs0_is_eq1(seed):
    """Gs = 0 reduces Eqs. (2)-(4) to the linear-gap recurrence Eq. (1) with g = -Ge."""
    rng = np.random.default_rng(200 + seed)
    for _ in range(20):
        m, n = int(rng.integers(1, 40)), int(rng.integers(1, 40))
        q = rng.integers(0, 20, m).astype(np.uint8)
        d = rng.integers(0, 20, n).astype(np.uint8)
        ge = int(rng.integers(1, 9))
        assert oracle.gotoh_score(q, d, B62, 0, ge) == linear_sw(q, d, B62, -ge)


def test_special_huge_gaps_is_kadane():
    rng = np.random.default_rng(300)
    for _ in range(40):
        m, n = int(rng.integers(1, 60)), int(rng.integers(1, 60))
        q = rng.integers(0, 20, m).astype(np.uint8)
        d = rng.integers(0, 20, n).astype(np.uint8)
        big = 11 * min(m, n) + 1  # any gap costs more than an alignment can gain
        assert oracle.gotoh_score(q, d, B62, big, 1) == ungapped_best(q, d, B62)


def test_special_single_residues_and_empty():
    for a in range(24):
        for b in range(24):
            v = oracle.gotoh_score(np.array([a], np.uint8), np.array([b], np.uint8), B62, 10, 2)
            assert v == max(0, int(B62[a, b]))
    e = np.zeros(0, np.uint8)
    assert oracle.gotoh_score(e, encode("WWW"), B62, 10, 2) == 0
    assert oracle.gotoh_score(encode("WWW"), e, B62, 10, 2) == 0


# ---------------------------------------------------------------- P5
def _rand_pair(rng, lo=1, hi=120):
    m, n = int(rng.integers(lo, hi)), int(rng.integers(lo, hi))
    return rng.integers(0, 20, m).astype(np.uint8), rng.integers(0, 20, n).astype(np.uint8)


def test_invariant_swap_bounds_self():
    rng = np.random.default_rng(400)
    pos = np.maximum(B62, 0)
    for _ in range(60):
        q, d = _rand_pair(rng)
        v = oracle.gotoh_score(q, d, B62, 10, 2)
        assert v >= 0
        assert v == oracle.gotoh_score(d, q, B62, 10, 2)          # BLOSUM62 symmetric
        lo = int(B62[np.ix_(q, d)].max()) if len(q) and len(d) else 0
        assert max(0, lo) <= v
        assert v <= min(int(pos[q].max(axis=1).sum()), int(pos[:, d].max(axis=0).sum()))
        self_v = oracle.gotoh_score(q, q, B62, 10, 2)
        assert self_v >= int(B62[q, q].sum())


def test_invariant_monotone_gaps_and_append():
    rng = np.random.default_rng(500)
    for _ in range(40):
        q, d = _rand_pair(rng, 2, 60)
        v = oracle.gotoh_score(q, d, B62, 10, 2)
        assert oracle.gotoh_score(q, d, B62, 11, 2) <= v
        assert oracle.gotoh_score(q, d, B62, 10, 3) <= v
        assert oracle.gotoh_score(q, d, B62, 9, 2) >= v
        extra = rng.integers(0, 20, int(rng.integers(1, 10))).astype(np.uint8)
        assert oracle.gotoh_score(np.concatenate([q, extra]), d, B62, 10, 2) >= v
        assert oracle.gotoh_score(q, np.concatenate([extra, d]), B62, 10, 2) >= v


def test_invariant_pad():
    """A PAD letter scoring <= 0 against everything never changes the score (reading R-12)."""
    S = np.full((25, 25), -4, dtype=np.int32)
    S[:24, :24] = B62
    rng = np.random.default_rng(600)
    for _ in range(40):
        q, d = _rand_pair(rng, 1, 50)
        v = oracle.gotoh_score(q, d, S, 10, 2)
        qp = np.concatenate([q, np.full(int(rng.integers(1, 9)), 24, np.uint8)])
        dp = np.concatenate([d, np.full(int(rng.integers(1, 9)), 24, np.uint8)])
        assert oracle.gotoh_score(qp, dp, S, 10, 2) == v


# ---------------------------------------------------------------- batch entry
def test_search_matches_pairs_and_procs():
    import swgen
    rng = np.random.default_rng(700)
    qc, qo = swgen.random_seqs(rng, 3, 1, 40)
    dc, do = swgen.random_seqs(rng, 37, 1, 50)
    ref = np.array([[oracle.gotoh_score(qc[qo[a]:qo[a + 1]], dc[do[b]:do[b + 1]], B62, 10, 2)
                     for b in range(37)] for a in range(3)], dtype=np.int32)
    np.testing.assert_array_equal(oracle.gotoh_search(qc, qo, dc, do, B62, 10, 2), ref)
    np.testing.assert_array_equal(oracle.gotoh_search(qc, qo, dc, do, B62, 10, 2, procs=3), ref)


def test_bad_code_raises():
    with pytest.raises(ValueError):
        oracle.gotoh_score(np.array([30], np.uint8), np.array([1], np.uint8), B62, 10, 2)


# ---------------------------------------------------------------------------
# Alignment: end cell, start cell and path of the best local
# alignment (oracle.gotoh_align), pinned against the exhaustive enumerator.

def _rand_case(rng, mmax=7, nmax=7, alpha=5):
    m, n = int(rng.integers(1, mmax + 1)), int(rng.integers(1, nmax + 1))
    q = rng.integers(0, alpha, size=m).astype(np.uint8)
    d = rng.integers(0, alpha, size=n).astype(np.uint8)
    S = rng.integers(-4, 7, size=(alpha, alpha)).astype(np.int32)   # asymmetric on purpose
    gs, ge = int(rng.integers(0, 6)), int(rng.integers(1, 4))
    return q, d, S, gs, ge


def test_align_end_and_path_vs_brute_force():
    """Score = the brute-force optimum; end = the optimal end with the smallest j,
    then smallest i (reading R-13); the returned path is one of the optimal
    alignments (chain of aligned pairs) and re-scores to the score."""
    rng = np.random.default_rng(505)
    for _ in range(250):
        q, d, S, gs, ge = _rand_case(rng)
        sc, qb, qe, db, de, ops = oracle.gotoh_align(q, d, S, gs, ge)
        best, chains = brute.brute_local_chains(q, d, S, gs, ge)
        assert sc == best
        if best == 0:
            assert (qb, qe, db, de, ops) == (-1, -1, -1, -1, [])
            continue
        ends = sorted({(c[-1][1], c[-1][0]) for c in chains})   # (j, i)
        assert (de, qe) == ends[0]
        pairs, qe2, de2 = brute.cigar_pairs(qb, db, ops)
        assert (qe2, de2) == (qe, de) and pairs[0] == (qb, db)
        assert pairs in set(chains)
        assert brute.score_cigar(q, d, qb, db, ops, S, gs, ge) == sc


def test_align_rescores_on_larger_inputs():
    """Beyond brute-force sizes: the path re-scores to the score and the score
    equals the linear-space scorer (two independent formulations)."""
    rng = np.random.default_rng(506)
    S = B62
    for _ in range(40):
        m, n = int(rng.integers(1, 120)), int(rng.integers(1, 160))
        q = rng.integers(0, 20, size=m).astype(np.uint8)
        d = rng.integers(0, 20, size=n).astype(np.uint8)
        if rng.random() < 0.5:  # plant a homologous stretch so paths have gaps
            k = min(m, n) // 2
            d[:k] = q[:k]
            d[k // 2] = (d[k // 2] + 3) % 20
        sc, qb, qe, db, de, ops = oracle.gotoh_align(q, d, S, 10, 2)
        assert sc == oracle.gotoh_score(q, d, S, 10, 2)
        if sc:
            assert brute.score_cigar(q, d, qb, db, ops, S, 10, 2) == sc
            assert ops[0] & 3 == 0 and ops[-1] & 3 == 0      # local alignments start and end on a pair


def test_align_fig1_linear_gaps():
    """Fig. 1 (L137-143) pair, ma +1 / mi -1 / linear g -2 (Gs = 0, Ge = 2): the
    local optimum 5 and a path that re-scores to it."""
    q, d, S = _dna("ACTTGTCCG"), _dna("ATTGTCAG"), _dna_matrix(1, -1)
    sc, qb, qe, db, de, ops = oracle.gotoh_align(q, d, S, 0, 2)
    assert sc == 5
    assert brute.score_cigar(q, d, qb, db, ops, S, 0, 2) == 5
