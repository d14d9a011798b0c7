"""Multi-GPU layer host logic: shard cut, dual-approx placement of
(query, shard) tasks, and the all-gather + assembly -- run with world_size 2
over gloo on CPU.  The per-rank scoring backend here is the CPU oracle (tests
may use it); on the GPU box the same dist.run() drives sw_search over NCCL.
The invariant: scores are identical for any world size and placement."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as tdist
import torch.multiprocessing as tmp

import oracle
import swgen
from oracle.blosum62 import blosum62 as ob62
from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist as swdist


def _workload():
    c = swgen.make_config("c1", n_db=160, q_lens=[37, 90, 12])
    return c


def _score_block_oracle(c, shards):
    def f(s, qs):
        sc, so = swdist.subset(c["dcodes"], c["doff"], shards[s])
        qc, qo = swdist.subset(c["qcodes"], c["qoff"], qs)
        return oracle.gotoh_search(qc, qo, sc, so, ob62(), 10, 2)
    return f


def test_shard_cut_partition_and_balance():
    c = swgen.make_config("c2", n_db=5000)
    lens = np.diff(c["doff"])
    for S in (1, 2, 3, 8):
        sh = swdist.shard_cut(c["doff"], S)
        allidx = np.sort(np.concatenate(sh))
        assert np.array_equal(allidx, np.arange(len(lens)))
        res = [int(lens[s].sum()) for s in sh]
        assert max(res) - min(res) <= 2 * lens.max()
        for s in sh:
            assert np.all(np.diff(s) > 0)


def test_subset_roundtrip():
    rng = np.random.default_rng(3)
    codes, off = swgen.random_seqs(rng, 50, 0, 30)
    idx = np.array([7, 3, 3, 49, 0])
    sc, so = swdist.subset(codes, off, idx)
    for k, i in enumerate(idx):
        assert np.array_equal(sc[so[k]:so[k + 1]], codes[off[i]:off[i + 1]])


def test_place_covers_every_task():
    c = swgen.make_config("c3", n_db=3000)
    ql = np.diff(c["qoff"])
    for g in (1, 2, 4, 8):
        sh = swdist.shard_cut(c["doff"], g)
        res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
        plan = swdist.place(ql, sh, res, g)
        seen = sorted((q, s) for r in range(g) for s, qs in swdist.local_blocks(plan, r) for q in qs)
        assert seen == sorted(plan.tasks)
        loads = np.zeros(g)
        for (q, s), o in zip(plan.tasks, plan.owner):
            loads[o] += swdist.gpu_task_time(ql[q], res[s])     # the calibrated model place() uses
        assert loads.max() == pytest.approx(plan.makespan)
        assert plan.makespan <= 2 * plan.lam * (1 + 1e-9)


def test_single_process_run_matches_oracle():
    c = _workload()
    ref = oracle.gotoh_search(c["qcodes"], c["qoff"], c["dcodes"], c["doff"], ob62(), 10, 2)
    sh = swdist.shard_cut(c["doff"], 3)
    res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
    plan = swdist.place(np.diff(c["qoff"]), sh, res, 1)
    got = swdist.run(plan, 0, len(c["qoff"]) - 1, len(c["doff"]) - 1, _score_block_oracle(c, sh))
    np.testing.assert_array_equal(got, ref)


def _worker(rank, world, port, n_shards, q):
    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    tdist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        c = _workload()
        sh = swdist.shard_cut(c["doff"], n_shards)
        res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
        plan = swdist.place(np.diff(c["qoff"]), sh, res, world)
        out = swdist.run(plan, rank, len(c["qoff"]) - 1, len(c["doff"]) - 1, _score_block_oracle(c, sh),
                         dist=tdist, assemble_on_all=True)
        q.put((rank, out))
    finally:
        tdist.destroy_process_group()


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.mark.parametrize("n_shards", [2, 5])
def test_gloo_world2_matches_single_process(n_shards):
    c = _workload()
    ref = oracle.gotoh_search(c["qcodes"], c["qoff"], c["dcodes"], c["doff"], ob62(), 10, 2)
    ctx = tmp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, n_shards, q)) for r in range(2)]
    for p in procs:
        p.start()
    outs = dict(q.get(timeout=240) for _ in procs)
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    for r in (0, 1):
        np.testing.assert_array_equal(outs[r], ref)


def test_place_hybrid_cpu_and_gpu_pes():
    """Hybrid placement: every (query, shard) task on exactly one
    PE; CPUs get work only when their rate makes it pay; makespan <= 2 lambda
    (Proposition 1)."""
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    rng = np.random.default_rng(4)
    offs = np.zeros(2001, dtype=np.int64)
    np.cumsum(rng.integers(10, 900, size=2000), out=offs[1:])
    shards = dist.shard_cut(offs, 8)
    res = [float((offs[idx + 1] - offs[idx]).sum()) for idx in shards]
    q_lens = [144, 567, 1000, 2504, 5478]
    slow = dist.place_hybrid(q_lens, shards, 4, 1, gpu_rate=6e12, cpu_rate=1e6, shard_residues=res)
    assert (slow.pe == 4).all()                      # CPUs far too slow: everything on the GPU
    mix = dist.place_hybrid(q_lens, shards, 16, 1, gpu_rate=1e11, cpu_rate=1e10, shard_residues=res)
    assert len(mix.pe) == len(q_lens) * 8 and set(mix.pe.tolist()) <= set(range(17))
    assert (mix.pe < 16).any() and (mix.pe == 16).any()
    loads = np.zeros(17)
    for t, p in enumerate(mix.pe):
        loads[p] += mix.p_cpu[t] if p < 16 else mix.p_gpu[t]
    assert abs(loads.max() - mix.makespan) < 1e-9 * max(1.0, mix.makespan)
    assert mix.makespan <= 2 * mix.lam * (1 + 1e-9)
    assert sorted(mix.cpu_tasks(0) + sum((mix.cpu_tasks(c) for c in range(1, 16)), []) + mix.gpu_tasks(0)) \
        == sorted(mix.tasks)


def test_place_hybrid_dp_variant():
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    rng = np.random.default_rng(5)
    offs = np.zeros(301, dtype=np.int64)
    np.cumsum(rng.integers(10, 900, size=300), out=offs[1:])
    shards = dist.shard_cut(offs, 4)
    res = [float((offs[idx + 1] - offs[idx]).sum()) for idx in shards]
    q_lens = [144, 567, 1000]
    g = dist.place_hybrid(q_lens, shards, 3, 1, gpu_rate=5e9, cpu_rate=1e9, shard_residues=res)
    d = dist.place_hybrid(q_lens, shards, 3, 1, gpu_rate=5e9, cpu_rate=1e9, shard_residues=res, variant="dp")
    assert len(d.pe) == len(g.pe) == 12
    assert d.makespan <= (1.5 + 0.25) * d.lam * (1 + 1e-9)
    assert d.makespan <= 2 * g.makespan


def _emulate_assemble(tabs, gathered, Q, N):
    """What sw_assemble computes (include/swdual.h), element by element."""
    blocks, rows, cols, _cap = tabs
    out = np.full((Q, N), -1, dtype=np.int32)
    for src_off, row_off, col_off, nr, nc in blocks:
        for i in range(nr):
            for k in range(nc):
                out[rows[row_off + i], cols[col_off + k]] = gathered[src_off + i * nc + k]
    return out


@pytest.mark.parametrize("world,shards", [(1, 1), (2, 8), (3, 5), (4, 16)])
def test_assembly_tables_match_assemble(world, shards):
    """The block tables handed to sw_assemble place every gathered score where
    dist.assemble (the host merge) does, and cover every (query, sequence)."""
    c = swgen.make_config("c3", n_db=300, q_lens=[50, 144, 30, 75, 9])
    ql = np.diff(c["qoff"])
    sh = swdist.shard_cut(c["doff"], shards)
    res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
    plan = swdist.place(ql, sh, res, world)
    tabs = swdist.assembly_tables(plan)
    cap = tabs[3]
    Q, N = len(ql), len(c["doff"]) - 1
    rng = np.random.default_rng(world * 10 + shards)
    flats = [rng.integers(0, 1000, size=cap).astype(np.int32) for _ in range(world)]
    gathered = np.concatenate(flats)
    ref = swdist.assemble(plan, Q, N, flats)
    got = _emulate_assemble(tabs, gathered, Q, N)
    assert (got >= 0).all()
    np.testing.assert_array_equal(got, ref)


def test_task_time_model_orders_by_padded_rows():
    """Calibrated GPU task times: strip-padded rows x residues
    / rate + a fixed share; a query costs as much as its strip-padded height."""
    t = swdist.gpu_task_time
    S = swdist.STRIP_ROWS
    assert t(S + 16, 1e6) == t(2 * S, 1e6)
    assert t(2 * S + 1, 1e6) > t(2 * S, 1e6)
    assert t(0, 1e6) == 0.0 and t(100, 0) == 0.0
    assert abs(t(9600, 1e8) - (9600 * 1e8 / swdist.RATE + swdist.T_TASK)) < 1e-12


@pytest.mark.parametrize("k", [1, 2, 3, 8])
def test_place_shards_one_search_per_gpu(k):
    """Shard tasks (every query against one shard): with S = k equal-residue
    shards the dual approximation gives each GPU exactly one shard (one search);
    every (query, shard) pair is covered once; the makespan is the largest
    shard's modelled time."""
    c = swgen.make_config("c3", n_db=4000)
    ql = np.diff(c["qoff"])
    sh = swdist.shard_cut(c["doff"], k)
    res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
    plan = swdist.place_shards(ql, sh, res, k)
    seen = sorted((q, s) for r in range(k) for s, qs in swdist.local_blocks(plan, r) for q in qs)
    assert seen == sorted((q, s) for q in range(len(ql)) for s in range(k))
    assert all(len(swdist.local_blocks(plan, r)) == 1 for r in range(k))
    per = [sum(swdist.gpu_task_time(m, res[s]) for m in ql) for s in range(k)]
    assert plan.makespan == pytest.approx(max(per))
