"""Independent reference computations used to PIN the oracle (tests only).

None of these shares code with oracle/ or with the product package; each is a
different formulation of what the paper defines:

* brute_local(): exhaustive enumeration of every local alignment (PAPER.md
  L127-136: score of an alignment = sum of its columns; the similarity is the
  maximal score) with affine gap runs costing Gs + k*Ge (Eqs. (3)-(4),
  L185-194; reading R-1).  An alignment of two substrings is an
  increasing chain of aligned pairs (i1<i2<..., j1<j2<...); between two
  consecutive pairs the skipped query residues form one gap run and the skipped
  subject residues another (interleaving them into more runs only adds opening
  costs).  Leading/trailing gaps never help, the empty alignment scores 0.
  The number of chains is C(m+n, m), so this is for m, n <= ~8.
* linear_sw(): Eq. (1) (L159-165) with a constant gap g, full (m+1)x(n+1)
  matrix -- the Gs = 0 special case of Eqs. (2)-(4).
* ungapped_best(): max over diagonals of the maximal-sum segment (Kadane) --
  what Eqs. (2)-(4) reduce to when every gap costs more than any alignment
  could gain.
* score_alignment(): score of a GIVEN alignment (two gapped strings of equal
  length), the sec. II.A definition (L127-134), for the Fig. 1 worked example.
"""
from __future__ import annotations


def brute_local(q, d, S, gs: int, ge: int) -> int:
    m, n = len(q), len(d)

    def gap(k: int) -> int:
        return gs + k * ge if k > 0 else 0

    best = 0
    stack = [(i, j, int(S[q[i]][d[j]])) for i in range(m) for j in range(n)]
    while stack:
        i, j, sc = stack.pop()
        if sc > best:
            best = sc
        for i2 in range(i + 1, m):
            gi = gap(i2 - i - 1)
            for j2 in range(j + 1, n):
                stack.append((i2, j2, sc - gi - gap(j2 - j - 1) + int(S[q[i2]][d[j2]])))
    return best


def linear_sw(q, d, S, g: int) -> int:
    """Eq. (1): H_ij = max(H_{i-1,j-1} + S_ij, H_{i,j-1} + g, H_{i-1,j} + g, 0); g <= 0."""
    m, n = len(q), len(d)
    H = [[0] * (n + 1) for _ in range(m + 1)]
    best = 0
    for i in range(1, m + 1):
        for j in range(1, n + 1):
            H[i][j] = max(H[i - 1][j - 1] + int(S[q[i - 1]][d[j - 1]]), H[i][j - 1] + g, H[i - 1][j] + g, 0)
            best = max(best, H[i][j])
    return best


def ungapped_best(q, d, S) -> int:
    m, n = len(q), len(d)
    best = 0
    for off in range(-(m - 1), n):
        run = 0
        for i in range(m):
            j = i + off
            if 0 <= j < n:
                run = max(0, run + int(S[q[i]][d[j]]))
                best = max(best, run)
    return best


def score_alignment(top: str, bottom: str, ma: int, mi: int, g: int) -> int:
    assert len(top) == len(bottom)
    s = 0
    for a, b in zip(top, bottom):
        if a == "-" or b == "-":
            s += g
        elif a == b:
            s += ma
        else:
            s += mi
    return s


def brute_local_chains(q, d, S, gs: int, ge: int):
    """Every optimal local alignment as its chain of aligned pairs, by the same
    exhaustive enumeration as brute_local(): (best, [chain, ...]) with chain a
    tuple of (i, j) pairs (0-based).  For m, n <= ~7."""
    m, n = len(q), len(d)

    def gap(k: int) -> int:
        return gs + k * ge if k > 0 else 0

    best, chains = 0, []
    stack = [(((i, j),), int(S[q[i]][d[j]])) for i in range(m) for j in range(n)]
    while stack:
        ch, sc = stack.pop()
        if sc > best:
            best, chains = sc, [ch]
        elif sc == best and sc > 0:
            chains.append(ch)
        i, j = ch[-1]
        for i2 in range(i + 1, m):
            gi = gap(i2 - i - 1)
            for j2 in range(j + 1, n):
                stack.append((ch + ((i2, j2),), sc - gi - gap(j2 - j - 1) + int(S[q[i2]][d[j2]])))
    return best, chains


def cigar_pairs(q_begin: int, d_begin: int, ops):
    """Aligned (i, j) pairs of a run-length op list (op 0 = M, 1 = I, 2 = D)."""
    i, j, out = q_begin, d_begin, []
    for c in ops:
        k, op = c >> 2, c & 3
        for _ in range(k):
            if op == 0:
                out.append((i, j)); i += 1; j += 1
            elif op == 1:
                i += 1
            else:
                j += 1
    return tuple(out), i - 1, j - 1


def score_cigar(q, d, q_begin: int, d_begin: int, ops, S, gs: int, ge: int) -> int:
    """Score of a GIVEN alignment in run-length form (sec. II.A: sum of
    the column scores; a gap run of length k costs Gs + k*Ge, reading R-1)."""
    i, j, s = q_begin, d_begin, 0
    for c in ops:
        k, op = c >> 2, c & 3
        if op == 0:
            for _ in range(k):
                s += int(S[q[i]][d[j]]); i += 1; j += 1
        elif op == 1:
            s -= gs + k * ge; i += k
        else:
            s -= gs + k * ge; j += k
    return s


def rule_alignment(q, d, S, gs: int, ge: int):
    """The best local alignment that reading R-13 selects, from the exhaustive
    enumeration (no DP matrices): among all optimal alignments, the end cell
    with the smallest j, then the smallest i; then, reading the alignment
    BACKWARDS from its end, the lexicographically smallest token sequence where
    at an aligned position the next token ranks STOP < M (diagonal) < D (gap in
    the query, E) < I (gap in the subject, F), and inside a gap run CLOSE (the
    run opens here) < EXTEND.  For Gs > 0 an optimal alignment has at most one
    I run and one D run between consecutive aligned pairs, so expanding every
    optimal chain of aligned pairs into its (one or two) gap orders lists them
    all.  Returns (score, q_begin, q_end, d_begin, d_end, ops) like
    oracle.gotoh_align, ops run-length (len << 2 | op), op 0 = M, 1 = I, 2 = D."""
    assert gs > 0, "the expansion below assumes Gs > 0"
    best, chains = brute_local_chains(q, d, S, gs, ge)
    if best == 0:
        return (0, -1, -1, -1, -1, [])
    end = min((c[-1][1], c[-1][0]) for c in chains)
    STOP, M, D, I = 0, 1, 2, 3
    CLOSE, EXT = 0, 1
    cands = []
    for c in chains:
        if (c[-1][1], c[-1][0]) != end:
            continue
        variants = [([], [])]           # (backward tokens, backward ops)
        for k in range(len(c) - 1, -1, -1):
            variants = [(t + [M], o + ["M"]) for t, o in variants]
            if k == 0:
                variants = [(t + [STOP], o) for t, o in variants]
                break
            di = c[k][0] - c[k - 1][0] - 1
            dj = c[k][1] - c[k - 1][1] - 1
            runD = ([D] + [EXT] * (dj - 1) + [CLOSE], ["D"] * dj) if dj else ([], [])
            runI = ([I] + [EXT] * (di - 1) + [CLOSE], ["I"] * di) if di else ([], [])
            orders = [(runD, runI), (runI, runD)] if (di and dj) else [(runD, runI)]
            variants = [(t + a[0] + b[0], o + a[1] + b[1]) for t, o in variants for a, b in orders]
        cands += [(t, o, c) for t, o in variants]
    tok, bops, c = min(cands, key=lambda x: x[0])
    fwd = bops[::-1]
    ops, run, prev = [], 0, None
    code = {"M": 0, "I": 1, "D": 2}
    for op in fwd + [None]:
        if op == prev:
            run += 1
            continue
        if prev is not None:
            ops.append((run << 2) | code[prev])
        prev, run = op, 1
    return (best, c[0][0], c[-1][0], c[0][1], c[-1][1], ops)
