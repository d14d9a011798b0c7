"""Multi-GPU layer: one process per GPU.

* shard_cut(): the length-sorted database is dealt snake-wise into S shards so
  every shard gets the same length mix and ~the same residues (the paper's
  very coarse-grained split of the work across PEs).
* place(): tasks are (query, shard) pairs -- the reading of "each task is the
  comparison of one [query] to the whole database" (L304-305) with the DB cut
  into shards (reading S-1); their GPU times come from a cell-rate
  model and the paper's dual approximation (sec. III, sw_schedule_dual)
  assigns them to the k GPUs (m = 0 CPUs on this box, reading S-6).
* run(): every rank scores its tasks with sw_search on its own device, then one
  collective -- an all-gather of the int32 score blocks (NCCL over NVLink on
  the GPU box, gloo in the CPU tests) -- after which every rank assembles
  scores[q][d] in the caller's order (the master's "merge", L527-528).
The database never moves after load; the only data-path exchange is the gather.
"""
from __future__ import annotations

from dataclasses import dataclass, field

import numpy as np

from .api import schedule_dual


def shard_cut(offsets, n_shards: int) -> list[np.ndarray]:
    """Caller indices of each shard (ascending).  Snake deal over the length order."""
    off = np.asarray(offsets, dtype=np.int64)
    n = len(off) - 1
    if n_shards < 1:
        raise ValueError("n_shards >= 1")
    lens = np.diff(off)
    order = np.argsort(-lens, kind="stable")
    pos = np.arange(n)
    rnd, k = pos // n_shards, pos % n_shards
    shard_of_rank = np.where(rnd % 2 == 0, k, n_shards - 1 - k)
    shard = np.empty(n, dtype=np.int64)
    shard[order] = shard_of_rank
    return [np.flatnonzero(shard == s) for s in range(n_shards)]


def subset(codes, offsets, idx):
    """(codes, offsets) of the sequences idx, in that order."""
    off = np.asarray(offsets, dtype=np.int64)
    idx = np.asarray(idx, dtype=np.int64)
    lens = off[idx + 1] - off[idx]
    new_off = np.zeros(len(idx) + 1, dtype=np.int64)
    np.cumsum(lens, out=new_off[1:])
    if len(idx) == 0:
        return np.zeros(0, np.uint8), new_off
    starts = off[idx]
    # gather residues
    rep = np.repeat(starts - new_off[:-1], lens)
    src = np.arange(int(new_off[-1]), dtype=np.int64) + rep
    return np.asarray(codes)[src], new_off


@dataclass
class Plan:
    n_gpus: int
    shards: list[np.ndarray]                 # caller indices per shard
    tasks: list[tuple[int, int]]             # (query, shard)
    owner: np.ndarray                        # task -> gpu
    makespan: float = 0.0
    lam: float = 0.0
    by_gpu: dict = field(default_factory=dict)  # gpu -> {shard: [queries]}


def place(q_lens, shards, shard_residues, n_gpus: int, rate: float = 1.0) -> Plan:
    """Dual-approximation placement of (query, shard) tasks on n_gpus GPUs.

    p_gpu(q, s) = m_q * residues(s) / rate  -- cells over a calibrated cell rate.
    """
    q_lens = [int(x) for x in q_lens]
    tasks = [(q, s) for q in range(len(q_lens)) for s in range(len(shards))]
    return _place(q_lens, shards, n_gpus, rate, tasks, [float(r) for r in shard_residues])


def _place(q_lens, shards, n_gpus, rate, tasks, res) -> Plan:
    p_gpu = np.array([q_lens[q] * res[s] / rate for q, s in tasks], dtype=np.float64)
    p_cpu = p_gpu * 1e6  # no CPU PEs on the B200 box (m = 0); unused when n_cpu = 0
    if len(tasks):
        pe, mk, lam = schedule_dual(p_cpu, p_gpu, 0, n_gpus)
    else:
        pe, mk, lam = np.zeros(0, np.int32), 0.0, 0.0
    plan = Plan(n_gpus=n_gpus, shards=shards, tasks=tasks, owner=np.asarray(pe, np.int64), makespan=mk, lam=lam)
    for g in range(n_gpus):
        plan.by_gpu[g] = {}
    for (q, s), g in zip(tasks, plan.owner):
        plan.by_gpu[int(g)].setdefault(s, []).append(q)
    return plan


def local_blocks(plan: Plan, rank: int):
    """Ordered list of (shard, queries) this rank scores; defines the flat layout."""
    d = plan.by_gpu.get(rank, {})
    return [(s, sorted(d[s])) for s in sorted(d)]


def flat_size(plan: Plan, rank: int) -> int:
    return sum(len(qs) * len(plan.shards[s]) for s, qs in local_blocks(plan, rank))


def assemble(plan: Plan, n_queries: int, n_seqs: int, flats) -> np.ndarray:
    """scores[q][d] from every rank's flat block list (caller order)."""
    out = np.zeros((n_queries, n_seqs), dtype=np.int32)
    for r in range(plan.n_gpus):
        f = np.asarray(flats[r])
        pos = 0
        for s, qs in local_blocks(plan, r):
            idx = plan.shards[s]
            blk = f[pos:pos + len(qs) * len(idx)].reshape(len(qs), len(idx))
            pos += len(qs) * len(idx)
            out[np.ix_(qs, idx)] = blk
    return out


def run(plan: Plan, rank: int, n_queries: int, n_seqs: int, score_block, dist=None, device=None,
        assemble_on_all: bool = False):
    """Score this rank's tasks with score_block(shard, queries) -> int32 [len(queries), len(shard)]
    (a torch tensor on `device` or a numpy array), then all-gather and assemble.

    dist: torch.distributed (initialised) or None for a single process.
    Returns scores [Q, N] (numpy) on rank 0 (or on all ranks if assemble_on_all), else None.
    """
    import torch
    blocks = local_blocks(plan, rank)
    parts = []
    for s, qs in blocks:
        b = score_block(s, qs)
        if not isinstance(b, torch.Tensor):
            b = torch.from_numpy(np.ascontiguousarray(b, dtype=np.int32))
        parts.append(b.reshape(-1).to(device) if device is not None else b.reshape(-1))
    world = plan.n_gpus
    sizes = [flat_size(plan, r) for r in range(world)]
    cap = max(sizes) if sizes else 0
    dev = device if device is not None else torch.device("cpu")
    mine = torch.zeros(max(cap, 1), dtype=torch.int32, device=dev)
    if parts:
        cat = torch.cat(parts)
        mine[:cat.numel()] = cat
    if dist is None or world == 1:
        flats = [mine.cpu().numpy()]
    else:
        gathered = torch.empty(world * mine.numel(), dtype=torch.int32, device=dev)
        dist.all_gather_into_tensor(gathered, mine)  # the single data-path collective
        if rank != 0 and not assemble_on_all:
            return None
        g = gathered.cpu().numpy().reshape(world, -1)
        flats = [g[r] for r in range(world)]
    return assemble(plan, n_queries, n_seqs, flats)
