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
    """(codes, offsets) of the sequences idx, in that order (sw_subset_host: a
    threaded host gather, no per-residue index array)."""
    import ctypes
    from ._lib import check, lib
    off = np.ascontiguousarray(offsets, dtype=np.int64)
    idx = np.ascontiguousarray(idx, dtype=np.int64)
    codes = np.ascontiguousarray(codes, dtype=np.uint8)
    new_off = np.zeros(len(idx) + 1, dtype=np.int64)
    n = ctypes.c_int64()
    vp = lambda a: a.ctypes.data_as(ctypes.c_void_p) if a.size else None  # noqa: E731
    check(lib().sw_subset_host(vp(codes), vp(off), len(off) - 1, vp(idx), len(idx), None, vp(new_off),
                               ctypes.byref(n)))
    out = np.empty(int(n.value), dtype=np.uint8)
    if len(idx):
        check(lib().sw_subset_host(vp(codes), vp(off), len(off) - 1, vp(idx), len(idx), vp(out), vp(new_off),
                                   ctypes.byref(n)))
    return out, new_off


@dataclass
class Plan:
    n_gpus: int
    shards: list[np.ndarray]                 # caller indices per shard
    tasks: list[tuple[int, int]]             # (query, shard)
    owner: np.ndarray                        # task -> gpu
    makespan: float = 0.0
    lam: float = 0.0
    by_gpu: dict = field(default_factory=dict)  # gpu -> {shard: [queries]}


# GPU time model of one (query, shard) task on a B200 (p_j from a
# calibrated rate).  The scoring kernel sweeps whole strips of STRIP_ROWS query
# rows (the query-pair geometry chosen for Swiss-Prot-like databases, G = 4 lanes
# x R = 32 rows), so a query of m residues costs ceil(m / STRIP_ROWS) * STRIP_ROWS
# rows -- which is why short queries run at a lower cell rate -- plus a per-task
# share of the search's fixed cost (launch tail, long-pair critical path).
# Calibrated on C3 in the k = 2 and k = 8 whole-shard layouts
# (profiles/r02_shard_probe.jsonl): t(k) = A / k + c with A = 1.115 s, c = 9.6 ms
# per 20-query search.
STRIP_ROWS = 128
RATE = 7.9e12          # strip-padded cells per second per B200
T_TASK = 4.8e-4        # seconds per task


def gpu_task_time(m: int, residues: float) -> float:
    rows = -(-int(m) // STRIP_ROWS) * STRIP_ROWS if m > 0 else 0
    return rows * float(residues) / RATE + (T_TASK if m > 0 and residues > 0 else 0.0)


def place(q_lens, shards, shard_residues, n_gpus: int, rate: float | None = None) -> Plan:
    """Dual-approximation placement of (query, shard) tasks on n_gpus GPUs.

    p_gpu(q, s) = gpu_task_time(m_q, residues(s)) (calibrated model), or
    m_q * residues(s) / rate when a plain cell rate is given.
    """
    q_lens = [int(x) for x in q_lens]
    tasks = [(q, s) for q in range(len(q_lens)) for s in range(len(shards))]
    return _place(q_lens, shards, n_gpus, rate, tasks, [float(r) for r in shard_residues])


def _place(q_lens, shards, n_gpus, rate, tasks, res) -> Plan:
    if rate is None:
        p_gpu = np.array([gpu_task_time(q_lens[q], res[s]) for q, s in tasks], dtype=np.float64)
    else:
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


def place_shards(q_lens, shards, shard_residues, n_gpus: int) -> Plan:
    """Dual-approximation placement of SHARD tasks: task s = every query against
    shard s (the paper's task is a query against the whole database, L304-305;
    with the database cut into shards the coarsest task is a shard with the whole
    query set).  One sw_search per task: with S = k equal-residue shards each GPU
    runs ONE search over 1/k of the database, the most efficient launch shape
    (measured: (query, shard) tasks on 4k shards scatter into ~30 small searches
    per GPU at k = 8 and run at a third of the single-search rate,
    profiles/r02_shard_probe.jsonl)."""
    q_lens = [int(x) for x in q_lens]
    res = [float(r) for r in shard_residues]
    p_gpu = np.array([sum(gpu_task_time(m, res[s]) for m in q_lens) for s in range(len(shards))], dtype=np.float64)
    if len(shards):
        pe, mk, lam = schedule_dual(p_gpu * 1e6, p_gpu, 0, n_gpus)
    else:
        pe, mk, lam = np.zeros(0, np.int32), 0.0, 0.0
    tasks = [(q, s) for s in range(len(shards)) for q in range(len(q_lens))]
    owner = np.array([int(pe[s]) for s in range(len(shards)) for _q in range(len(q_lens))], dtype=np.int64)
    plan = Plan(n_gpus=n_gpus, shards=shards, tasks=tasks, owner=owner, makespan=mk, lam=lam)
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


def assembly_tables(plan: Plan):
    """Block tables of the gathered buffer for sw_assemble (every rank's flat block
    list, rank r's at offset r * cap, cap = the largest rank's flat size):
    (blocks int64[n][5] = src_off, row_off, col_off, n_rows, n_cols; rows int32;
    cols int64; cap).  A shard's column list is stored once."""
    world = plan.n_gpus
    cap = max([flat_size(plan, r) for r in range(world)] + [1])
    blocks, rows, cols, col_off = [], [], [], {}
    n_rows = 0
    n_cols = 0
    for r in range(world):
        pos = r * cap
        for s, qs in local_blocks(plan, r):
            idx = plan.shards[s]
            if s not in col_off:
                col_off[s] = n_cols
                cols.append(np.asarray(idx, dtype=np.int64))
                n_cols += len(idx)
            blocks.append((pos, n_rows, col_off[s], len(qs), len(idx)))
            rows.append(np.asarray(qs, dtype=np.int32))
            n_rows += len(qs)
            pos += len(qs) * len(idx)
    cat = lambda xs, dt: np.concatenate(xs).astype(dt) if xs else np.zeros(0, dt)  # noqa: E731
    return (np.array(blocks, dtype=np.int64).reshape(-1, 5), cat(rows, np.int32), cat(cols, np.int64), cap)


class ShardedSearch:
    """One rank's part of the multi-GPU search; bench.py and the
    tests run THIS code path.

    Setup (untimed, like a resident search service): the DB is cut into
    n_shards snake-dealt shards of equal residues (default one per GPU); the
    tasks -- whole shards with every query (tasks="shard", default) or (query,
    shard) pairs (tasks="pair") -- are placed by the dual approximation
    (sw_schedule_dual, calibrated task times); this rank loads the shards its
    tasks reference and prepares one sw_search per (shard, query list) block
    into a flat device buffer.
    step(): the rank's searches, then -- the single data-path exchange -- the
    all-gather of the flat blocks (NCCL over NVLink; gloo with host staging for
    functional runs), then on rank 0 sw_assemble merges them into scores[Q][N]
    in the caller's order (the master's merge).  With one
    GPU and one shard the search writes the full matrix directly.
    """

    def __init__(self, handle, dcodes, doff, qcodes, qoff, matrix, gap_open=10, gap_extend=2, rank=0, world=1,
                 n_shards=None, pg=None, backend="nccl", alphabet_size=24, rate=None, tasks="shard"):
        import torch
        self.h, self.rank, self.world, self.pg, self.backend = handle, rank, world, pg, backend
        self.matrix, self.gs, self.ge = matrix, gap_open, gap_extend
        doff = np.asarray(doff, dtype=np.int64)
        qoff = np.asarray(qoff, dtype=np.int64)
        self.Q, self.N = len(qoff) - 1, len(doff) - 1
        n_shards = n_shards or world
        self.shards = shard_cut(doff, n_shards)
        lens = np.diff(doff)
        res = [int(lens[s].sum()) for s in self.shards]
        if tasks == "shard":
            self.plan = place_shards(np.diff(qoff), self.shards, res, world)
        else:  # (query, shard) tasks
            self.plan = place(np.diff(qoff), self.shards, res, world, rate=rate)
        self.blocks = local_blocks(self.plan, rank)
        dev = torch.device("cuda", handle.device)
        self.dev = dev
        self.dbs = {}
        for s, _qs in self.blocks:
            self.dbs[s] = handle.load_db(*subset(dcodes, doff, self.shards[s]), alphabet_size=alphabet_size)
        tabs = assembly_tables(self.plan)
        self.cap = tabs[3]
        single = world == 1 and len(self.blocks) == 1 and len(self.blocks[0][1]) == self.Q \
            and np.array_equal(self.shards[self.blocks[0][0]], np.arange(self.N))
        self.flat = torch.zeros(self.cap, dtype=torch.int32, device=dev)
        self.full = None
        self.asm = None
        if single:
            self.full = self.flat[:self.Q * self.N].view(self.Q, self.N)
        elif rank == 0:
            self.full = torch.zeros((self.Q, self.N), dtype=torch.int32, device=dev)
            self.asm = handle.assembly(tabs[0], tabs[1], tabs[2], self.Q, self.N)
        self.gathered = (torch.empty(world * self.cap, dtype=torch.int32, device=dev) if world > 1
                         else self.flat)
        self.jobs = []
        pos = 0
        for s, qs in self.blocks:
            qc, qo = subset(qcodes, qoff, qs)
            n = len(self.shards[s])
            self.jobs.append((s, qs, qc, qo, self.flat[pos:pos + len(qs) * n].view(len(qs), n)))
            pos += len(qs) * n

    def search_local(self, stream=None, host_out=None):
        for k, (s, _qs, qc, qo, view) in enumerate(self.jobs):
            out = view if host_out is None else host_out[k]
            self.h.search(qc, qo, self.dbs[s], self.matrix, self.gs, self.ge, out=out, stream=stream)

    def exchange(self, stream=None):
        """All-gather of the flat blocks, then rank 0's merge (no-op at N = 1, one shard)."""
        import torch
        if self.world > 1:
            if self.backend == "nccl":
                self.pg.all_gather_into_tensor(self.gathered, self.flat)
            else:  # gloo: host staging (functional runs only)
                torch.cuda.synchronize(self.dev)
                g = torch.empty(self.world * self.cap, dtype=torch.int32)
                self.pg.all_gather_into_tensor(g, self.flat.cpu())
                self.gathered.copy_(g)
        if self.asm is not None:
            self.asm(self.gathered, self.full, stream=stream)

    def step(self, stream=None):
        """One pass of the whole path; returns the device scores[Q][N] on rank 0 (else None)."""
        self.search_local(stream)
        self.exchange(stream)
        return self.full

    def local_cells(self) -> float:
        return float(sum(float(np.diff(qo).sum()) * float(self.dbs[s].info()["n_residues"])
                         for s, _q, _qc, qo, _v in self.jobs))


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


# ---------------------------------------------------------------------------
# Hybrid SWDUAL on one box: the paper's setting of "m CPUs and
# k GPUs" with host cores as CPU-type PEs.  Every task
# (query, shard) has a CPU time and a GPU time from calibrated cell rates; the
# dual approximation (sw_schedule_dual) places it; the GPU tasks run through
# sw_search while the CPU PEs run theirs concurrently through sw_search_cpu
# (one host thread per PE).  Opt-in: plain searches never touch the CPU path.

@dataclass
class HybridPlan:
    shards: list[np.ndarray]
    tasks: list[tuple[int, int]]             # (query, shard)
    pe: np.ndarray                           # task -> PE (0..n_cpus-1 CPUs, then GPUs)
    n_cpus: int
    n_gpus: int
    makespan: float
    lam: float
    p_cpu: np.ndarray
    p_gpu: np.ndarray

    def cpu_tasks(self, c: int):
        return [t for t, p in zip(self.tasks, self.pe) if p == c]

    def gpu_tasks(self, g: int = 0):
        return [t for t, p in zip(self.tasks, self.pe) if p == self.n_cpus + g]


def place_hybrid(q_lens, shards, n_cpus: int, n_gpus: int, gpu_rate: float, cpu_rate: float,
                 shard_residues=None, variant: str = "greedy") -> HybridPlan:
    """Tasks (query, shard) with p = cells / rate on each PE type (reading S-1/S-2),
    placed by the dual approximation on n_cpus CPU PEs + n_gpus GPUs.

    gpu_rate / cpu_rate: cells per second, a scalar or one value per query (the
    GPU's rate depends on the query length -- short queries fill its lanes
    worse -- so p_cpu / p_gpu differs between tasks, which is what the
    knapsack of the dual approximation orders by, L370-387)."""
    if shard_residues is None:
        raise ValueError("shard_residues required")
    tasks = [(q, s) for q in range(len(q_lens)) for s in range(len(shards))]
    cells = np.array([float(q_lens[q]) * float(shard_residues[s]) for q, s in tasks], dtype=np.float64)
    qi = np.array([q for q, _ in tasks], dtype=np.int64)
    gr = np.broadcast_to(np.asarray(gpu_rate, dtype=np.float64), (len(q_lens),))[qi] if tasks else np.zeros(0)
    cr = np.broadcast_to(np.asarray(cpu_rate, dtype=np.float64), (len(q_lens),))[qi] if tasks else np.zeros(0)
    p_cpu, p_gpu = cells / cr, cells / gr
    if tasks:
        pe, mk, lam = schedule_dual(p_cpu, p_gpu, n_cpus, n_gpus, variant=variant)
    else:
        pe, mk, lam = np.zeros(0, np.int32), 0.0, 0.0
    return HybridPlan(shards, tasks, np.asarray(pe, np.int64), n_cpus, n_gpus, mk, lam, p_cpu, p_gpu)


class HybridDB:
    """A database cut into shards, resident both on the GPU (one sw_db per shard,
    loaded once) and on the host (for the CPU PEs)."""

    def __init__(self, handle, db_codes, db_offsets, n_shards: int = 8, alphabet_size: int = 24):
        self.handle = handle
        self.alphabet_size = alphabet_size
        self.db_offsets = np.ascontiguousarray(db_offsets, dtype=np.int64)
        self.n_seqs = len(self.db_offsets) - 1
        self.shards = shard_cut(self.db_offsets, n_shards)
        self.host = [subset(db_codes, self.db_offsets, idx) for idx in self.shards]
        self.gpu = [handle.load_db(c, o, alphabet_size=alphabet_size) for c, o in self.host]
        self.residues = [float(o[-1] - o[0]) for _, o in self.host]

    def plan(self, q_lens, n_cpus: int, gpu_rate: float, cpu_rate: float, variant: str = "greedy") -> HybridPlan:
        return place_hybrid(q_lens, self.shards, n_cpus, 1, gpu_rate, cpu_rate, shard_residues=self.residues,
                            variant=variant)

    def search(self, q_codes, q_offsets, matrix, gap_open=10, gap_extend=2, n_cpus: int = 4,
               gpu_rate: float = 6.5e12, cpu_rate: float = 3.0e9, plan: HybridPlan | None = None):
        """scores int32[Q, N] (caller order) from the GPU + n_cpus host PEs.

        Returns (scores, info): the plan and the wall time each PE took."""
        import threading
        import time

        from .api import search_cpu

        q_codes = np.ascontiguousarray(q_codes, dtype=np.uint8)
        q_offsets = np.ascontiguousarray(q_offsets, dtype=np.int64)
        nq = len(q_offsets) - 1
        if plan is None:
            plan = self.plan(np.diff(q_offsets), n_cpus, gpu_rate, cpu_rate)
        out = np.zeros((nq, self.n_seqs), dtype=np.int32)
        info = {"plan": plan, "cpu_s": [0.0] * plan.n_cpus, "gpu_s": 0.0}

        def groups(tasks):
            by = {}
            for q, s in tasks:
                by.setdefault(s, []).append(q)
            return [(s, sorted(qs)) for s, qs in sorted(by.items())]

        def cpu_pe(c):
            t0 = time.perf_counter()
            for s, qs in groups(plan.cpu_tasks(c)):
                qc, qo = subset(q_codes, q_offsets, qs)
                blk = search_cpu(qc, qo, self.host[s][0], self.host[s][1], matrix, gap_open, gap_extend,
                                 alphabet_size=self.alphabet_size, n_threads=1)
                out[np.ix_(qs, self.shards[s])] = blk
            info["cpu_s"][c] = time.perf_counter() - t0

        threads = [threading.Thread(target=cpu_pe, args=(c,)) for c in range(plan.n_cpus)]
        for t in threads:
            t.start()
        t0 = time.perf_counter()
        for s, qs in groups(plan.gpu_tasks(0)):
            qc, qo = subset(q_codes, q_offsets, qs)
            blk = np.zeros((len(qs), len(self.shards[s])), dtype=np.int32)
            self.handle.search(qc, qo, self.gpu[s], matrix, gap_open, gap_extend, out=blk)
            out[np.ix_(qs, self.shards[s])] = blk
        info["gpu_s"] = time.perf_counter() - t0
        for t in threads:
            t.join()
        return out, info
