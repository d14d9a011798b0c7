"""Dual-approximation scheduler (sec. III) through the C ABI.

Several schedules are valid, so the tests check what the paper fixes:
Proposition 1 (makespan <= 2*lambda, L397-467), the 2-approximation against a
brute-force optimum on tiny instances, validity, determinism, and the m = 0
CPU case used on the B200 box (reading S-6).
"""
import itertools

import numpy as np
import pytest

from paper_conf_icpp_kedad_sidhoummmmt14_b200 import schedule_dual, SWError


def loads(pe, pc, pg, m, k):
    L = np.zeros(m + k)
    for j, p in enumerate(pe):
        L[p] += pc[j] if p < m else pg[j]
    return L


def brute_opt(pc, pg, m, k):
    n = len(pc)
    best = np.inf
    for assign in itertools.product(range(m + k), repeat=n):
        best = min(best, loads(assign, pc, pg, m, k).max())
    return best


@pytest.mark.parametrize("seed", range(8))
def test_two_approx_vs_brute_force(seed):
    rng = np.random.default_rng(seed)
    for _ in range(25):
        n = int(rng.integers(1, 7))
        m = int(rng.integers(0, 3))
        k = int(rng.integers(1 if m == 0 else 0, 3))
        if m + k == 0 or m + k > 3:
            continue
        pg = rng.uniform(0.1, 10.0, n)
        pc = pg * rng.uniform(0.5, 30.0, n)  # most tasks are accelerated on GPUs (L497-499)
        pe, mk, lam = schedule_dual(pc, pg, m, k)
        assert np.all((pe >= 0) & (pe < m + k))
        L = loads(pe, pc, pg, m, k)
        assert mk == pytest.approx(L.max())
        assert mk <= 2 * lam * (1 + 1e-9)                     # Proposition 1
        opt = brute_opt(pc, pg, m, k)
        assert lam <= opt * (1 + 2e-4) + 1e-12                  # any lambda >= OPT is accepted
        assert mk <= 2 * opt * (1 + 2e-4) + 1e-12               # 2-approximation


def test_gpu_only_is_lpt_quality():
    rng = np.random.default_rng(9)
    for _ in range(50):
        n, k = int(rng.integers(1, 40)), int(rng.integers(1, 9))
        pg = rng.uniform(1, 100, n)
        pe, mk, lam = schedule_dual(pg * 5, pg, 0, k)
        assert np.all((pe >= 0) & (pe < k))
        L = loads(pe, pg * 5, pg, 0, k)
        lb = max(pg.max(), pg.sum() / k)
        assert mk == pytest.approx(L.max())
        assert mk <= (4.0 / 3.0) * lb + 1e-9 or mk <= 2 * lb    # LPT bound w.r.t. the lower bound
        assert mk <= 2 * lam * (1 + 1e-9)


def test_deterministic_and_edges():
    pc = np.array([5.0, 4.0, 3.0, 2.0, 1.0])
    pg = np.array([1.0, 1.0, 2.0, 2.0, 0.5])
    a = schedule_dual(pc, pg, 2, 2)
    b = schedule_dual(pc, pg, 2, 2)
    assert np.array_equal(a[0], b[0]) and a[1] == b[1]
    pe, mk, lam = schedule_dual([], [], 1, 1)
    assert len(pe) == 0 and mk == 0
    # CPU-only
    pe, mk, _ = schedule_dual([3.0, 3.0, 2.0], [1.0, 1.0, 1.0], 2, 0)
    assert set(pe.tolist()) <= {0, 1} and mk == pytest.approx(5.0)
    with pytest.raises(SWError):
        schedule_dual([1.0], [1.0], 0, 0)
    with pytest.raises(SWError):
        schedule_dual([-1.0], [1.0], 1, 1)


def test_task_longer_than_lambda_goes_to_other_side():
    # task 0 is hopeless on the CPU, task 1 on the GPU: a 1+1 box must split them
    pe, mk, lam = schedule_dual([100.0, 1.0], [1.0, 100.0], 1, 1)
    assert pe.tolist() == [1, 0] and mk == pytest.approx(1.0)


@pytest.mark.parametrize("seed", range(6))
def test_dp_variant_vs_brute_force(seed):
    """DP-knapsack variant (reading S-8): every lambda >= OPT is
    accepted and the schedule ends by (3/2 + 1/(4k)) lambda, so it is within that
    factor of the brute-force optimum."""
    rng = np.random.default_rng(100 + seed)
    for _ in range(25):
        n = int(rng.integers(1, 7))
        m = int(rng.integers(0, 3))
        k = int(rng.integers(1, 3))
        if m + k > 3:
            continue
        pg = rng.uniform(0.1, 10.0, n)
        pc = pg * rng.uniform(0.5, 30.0, n)
        pe, mk, lam = schedule_dual(pc, pg, m, k, variant="dp")
        assert np.all((pe >= 0) & (pe < m + k))
        L = loads(pe, pc, pg, m, k)
        assert mk == pytest.approx(L.max())
        bound = 1.5 + 0.25 / k
        assert mk <= bound * lam * (1 + 1e-9)
        opt = brute_opt(pc, pg, m, k)
        assert lam <= opt * (1 + 2e-4) + 1e-12
        assert mk <= bound * opt * (1 + 2e-4) + 1e-12


def test_dp_variant_not_worse_on_average():
    """On random hybrid instances the DP variant's makespans are on average no
    worse than the greedy 2-approximation's (same binary search)."""
    rng = np.random.default_rng(77)
    ratios = []
    for _ in range(40):
        n, m, k = int(rng.integers(8, 30)), int(rng.integers(1, 6)), int(rng.integers(1, 3))
        pg = rng.uniform(1, 20, n)
        pc = pg * rng.uniform(2, 20, n)
        _, mg, _ = schedule_dual(pc, pg, m, k)
        _, md, _ = schedule_dual(pc, pg, m, k, variant="dp")
        ratios.append(md / mg)
    assert np.mean(ratios) <= 1.0 + 1e-9


def test_dp_variant_size_limit():
    pg = np.ones(5000)
    with pytest.raises(SWError):
        schedule_dual(pg * 3, pg, 64, 8, variant="dp")
