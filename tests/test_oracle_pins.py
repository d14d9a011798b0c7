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


def test_align_tie_breaks_vs_enumeration():
    """The WHOLE returned alignment -- end cell, start cell and every op, i.e.
    the traceback's tie-breaks of reading R-13 (diagonal > E > F at an aligned
    position, opening > extending inside a gap, stop at the first zero prefix) --
    equals the one brute.rule_alignment selects by lexicographic order over the
    exhaustively enumerated optimal alignments (no DP).  Small alphabets and
    matrices with many equal entries make ties frequent."""
    rng = np.random.default_rng(507)
    n_ties = 0
    for _ in range(400):
        alpha = int(rng.integers(2, 4))
        m, n = int(rng.integers(1, 7)), int(rng.integers(1, 7))
        q = rng.integers(0, alpha, size=m).astype(np.uint8)
        d = rng.integers(0, alpha, size=n).astype(np.uint8)
        S = rng.choice([-2, -1, 0, 1, 2, 3], size=(alpha, alpha)).astype(np.int32)
        gs, ge = int(rng.integers(1, 4)), int(rng.integers(0, 3))
        got = oracle.gotoh_align(q, d, S, gs, ge)
        exp = brute.rule_alignment(q, d, S, gs, ge)
        assert got == exp, (q.tolist(), d.tolist(), S.tolist(), gs, ge, got, exp)
        best, chains = brute.brute_local_chains(q, d, S, gs, ge)
        n_ties += len(chains) > 1
    assert n_ties > 100   # the sample really exercises the tie-breaks


def _abcxy_matrix():
    """a b c x y: a/a = c/c = 10, a/b = b/a = 9, every other pair -10."""
    S = np.full((5, 5), -10, dtype=np.int32)
    S[0, 0] = S[2, 2] = 10
    S[0, 1] = S[1, 0] = 9
    return S


@pytest.mark.parametrize("case", [
    # (query, subject, Gs, Ge, expected (score, qb, qe, db, de), expected ops); derivations in the docstring
    ("ac", "abc", 1, 0, (19, 0, 1, 1, 2), ["2M"]),
    ("axc", "ayc", 1, 1, (16, 0, 2, 0, 2), ["1M", "1I", "1D", "1M"]),
    ("ac", "aaxc", 1, 0, (19, 0, 1, 1, 3), ["1M", "1D", "1M"]),
    ("aaxc", "ac", 1, 0, (19, 1, 3, 0, 1), ["1M", "1I", "1M"]),
    ("a", "aa", 1, 1, (10, 0, 0, 0, 0), ["1M"]),
    ("aa", "a", 1, 1, (10, 0, 0, 0, 0), ["1M"]),
])
def test_align_tie_breaks_hand_derived(case):
    """Hand-derived cases, matrix _abcxy_matrix():
    1. diagonal vs E at an aligned position.  q=ac, d=abc, Gs 1, Ge 0: a-b then c-c
       = 9 + 10 = 19, and a-a, gap over b, c-c = 10 - 1 + 10 = 19; no ungapped c pairs
       better.  End (q1, d2) is unique; back at H(q0, d1) both the diagonal (a-b) and E
       (b against a gap) reach 9: the diagonal wins -> q0-d1, q1-d2: ops 2M, db = 1.
    2. E vs F.  q=axc, d=ayc, Gs 1, Ge 1: a-a, x against a gap, y against a gap, c-c =
       20 - 2 - 2 = 16 (aligning x-y gives 10).  At H(q1, d1) H = E = F = 6 and the
       diagonal (x-y) does not reach it: E first, so backwards the D run (y) comes
       before the I run (x): forward M I D M.
    3. open vs extend inside an E run.  q=ac, d=aaxc, Gs 1, Ge 0: q0 against d1 then a
       one-residue gap (x), or q0 against d0 then a two-residue gap (a, x): both 19.
       At E(q0, d2) opening from H(q0, d1) = 10 ties extending E(q0, d1) = 9: open ->
       q0-d1, D, q1-d3: ops M D M, db = 1.
    4. the same inside an F run (query and subject swapped): ops M I M, qb = 1.
    5. end-cell tie in j: q=a, d=aa: 10 at (q0, d0) and (q0, d1): smallest j, d0.
    6. end-cell tie in i: q=aa, d=a: 10 at (q0, d0) and (q1, d0): smallest i, q0.
    (Stopping at the first zero prefix is covered by the enumeration test above.)
    """
    q, d, gs, ge, five, ops = case
    S = _abcxy_matrix()
    enc = {"a": 0, "b": 1, "c": 2, "x": 3, "y": 4}
    qa = np.array([enc[x] for x in q], np.uint8)
    da = np.array([enc[x] for x in d], np.uint8)
    code = {"M": 0, "I": 1, "D": 2}
    exp_ops = [(int(o[:-1]) << 2) | code[o[-1]] for o in ops]
    got = oracle.gotoh_align(qa, da, S, gs, ge)
    assert got == five + (exp_ops,)
    assert brute.rule_alignment(qa, da, S, gs, ge) == got
