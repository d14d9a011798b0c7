"""CPU-type processing element of the hybrid SWDUAL (
sw_search_cpu, csrc/cpu_striped.cpp) against the oracle, bit-exact.  Host only
(no GPU): the striped AVX2 int16 kernel, its lazy-F pass across lane
boundaries, saturation -> int32 re-score, random asymmetric matrices with
frequent ties, Gs = 0 (Eq. (1)), and the ragged query lengths around the
16-lane segment boundaries."""
import ctypes

import numpy as np
import pytest

import oracle
from oracle.blosum62 import blosum62 as oracle_b62


def _pkg():
    import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
    return sw


def _seqs(lengths, rng, alpha):
    lens = np.asarray(lengths, dtype=np.int64)
    off = np.zeros(len(lens) + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    return rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8), off


def cpu_scores(qc, qo, dc, do, S, gs, ge, alpha, threads=2):
    sw = _pkg()
    return sw.search_cpu(qc, qo, dc, do, S, gs, ge, alphabet_size=alpha, n_threads=threads)


@pytest.mark.parametrize("alpha,gs,ge", [(4, 3, 1), (4, 0, 2), (3, 0, 0), (6, 5, 1), (24, 10, 2), (5, 0, 1)])
def test_cpu_pe_vs_oracle(alpha, gs, ge):
    rng = np.random.default_rng(300 + 11 * alpha + gs + ge)
    S = oracle_b62().astype(np.int8) if alpha == 24 else rng.integers(-4, 6, size=(alpha, alpha)).astype(np.int8)
    ql = [1, 2, 15, 16, 17, 31, 32, 33, 100, 255, 257]
    dl = list(rng.integers(0, 400, size=60)) + [0, 1, 2]
    qc, qo = _seqs(ql, rng, min(alpha, 20))
    dc, do = _seqs(dl, rng, min(alpha, 20))
    got = cpu_scores(qc, qo, dc, do, S, gs, ge, alpha)
    ref = oracle.gotoh_search(qc, qo, dc, do, S.astype(np.int32), gs, ge)
    np.testing.assert_array_equal(got, ref)


def test_cpu_pe_saturation_rescore():
    """Self-hits of a W-rich query exceed int16: flagged and re-scored in int32."""
    rng = np.random.default_rng(8)
    W = 17  # 'W' in NCBI order, S(W,W) = 11
    q = np.full(4000, W, dtype=np.uint8)
    q[::7] = rng.integers(0, 20, size=len(q[::7]))
    d = np.concatenate([q[50:3950], rng.integers(0, 20, size=50).astype(np.uint8)])
    qo = np.array([0, len(q)], dtype=np.int64)
    do = np.array([0, len(d), len(d) + 40], dtype=np.int64)
    dc = np.concatenate([d, rng.integers(0, 20, size=40).astype(np.uint8)])
    got = cpu_scores(q, qo, dc, do, oracle_b62().astype(np.int8), 10, 2, 24)
    ref = oracle.gotoh_search(q, qo, dc, do, oracle_b62(), 10, 2)
    assert ref[0, 0] > 32767
    np.testing.assert_array_equal(got, ref)


def test_cpu_pe_errors_and_threads():
    sw = _pkg()
    rng = np.random.default_rng(2)
    qc, qo = _seqs([20, 40], rng, 20)
    dc, do = _seqs(list(rng.integers(1, 200, size=300)), rng, 20)
    S = oracle_b62().astype(np.int8)
    a = cpu_scores(qc, qo, dc, do, S, 10, 2, 24, threads=1)
    b = cpu_scores(qc, qo, dc, do, S, 10, 2, 24, threads=7)
    np.testing.assert_array_equal(a, b)
    with pytest.raises(sw.SWError):
        sw.search_cpu(qc, qo, dc, do, S, -1, 2, alphabet_size=24)
    bad = dc.copy()
    bad[3] = 24
    with pytest.raises(sw.SWError):
        sw.search_cpu(qc, qo, bad, do, S, 10, 2, alphabet_size=24)
    assert sw.search_cpu(qc[:0], np.zeros(1, np.int64), dc, do, S, 10, 2).shape == (0, len(do) - 1)
