"""The multi-GPU path on the one GPU this box has.

* bench.py's own N > 1 step (dist.ShardedSearch: shard cut, dual-approximation
  placement, per-rank sw_search, all-gather, rank 0's sw_assemble into caller
  order) run by torchrun with 2 ranks sharing the device over gloo; rank 0's
  assembled matrix is checked against the oracle (every sequence of C1).
* sw_assemble itself on a random layout vs the host merge (dist.assemble).
* the placement model (calibrated task times) against the measured per-rank
  device time of the same placement's searches.
"""
import json
import os
import socket
import subprocess
import sys

import numpy as np
import pytest

import swgen

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.mark.parametrize("workload,verify", [("c1", 1000), ("c4", 40)])
def test_bench_two_ranks_functional(workload, verify):
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node=2",
           "--master-addr=127.0.0.1", f"--master-port={_free_port()}", os.path.join(ROOT, "bench.py"),
           "--gpus", "2", "--steps", "1", "--warmup", "3", "--e2e-steps", "1", "--dist-backend", "gloo",
           "--workload", workload, "--verify", str(verify), "--no-cpu-baseline"]
    r = subprocess.run(cmd, cwd=ROOT, capture_output=True, text=True, timeout=900)
    assert r.returncode == 0, r.stderr[-3000:]
    line = json.loads([ln for ln in r.stdout.splitlines() if ln.startswith("{")][-1])
    assert line["n_gpus"] == 2 and line["verified"] is True
    assert line["config"]["shards"] == 2


def test_assemble_kernel_matches_host_merge():
    import torch
    import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    c = swgen.make_config("c3", n_db=5000)
    ql = np.diff(c["qoff"])
    sh = dist.shard_cut(c["doff"], 24)
    res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
    plan = dist.place(ql, sh, res, 6)
    blocks, rows, cols, cap = dist.assembly_tables(plan)
    Q, N = len(ql), len(c["doff"]) - 1
    rng = np.random.default_rng(4)
    flats = [rng.integers(0, 1 << 30, size=cap).astype(np.int32) for _ in range(6)]
    with sw.Handle(0) as h:
        asm = h.assembly(blocks, rows, cols, Q, N)
        src = torch.from_numpy(np.concatenate(flats)).cuda()
        out = torch.full((Q, N), -1, dtype=torch.int32, device="cuda")
        asm(src, out)
        torch.cuda.synchronize()
        got = out.cpu().numpy()
        with pytest.raises(sw.SWError):
            asm(src[:10], out)          # shorter than the blocks
    np.testing.assert_array_equal(got, dist.assemble(plan, Q, N, flats))


@pytest.mark.parametrize("k", [2, 4, 8])
def test_placement_model_vs_measured(k):
    """Modelled makespan of the dual-approximation placement (C3, k whole-shard
    tasks, the bench's N-GPU layout) is within 10 % of the measured max per-rank
    device time when each rank's search is run on this GPU one after the other."""
    import torch
    import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    c = swgen.make_config("c3")
    ql = np.diff(c["qoff"])
    sh = dist.shard_cut(c["doff"], k)
    res = [int(np.diff(c["doff"])[s].sum()) for s in sh]
    plan = dist.place_shards(ql, sh, res, k)
    times = []
    with sw.Handle(0) as h:
        dbs = {s: h.load_db(*dist.subset(c["dcodes"], c["doff"], sh[s])) for s in range(len(sh))}
        jobs = {r: [(s, *dist.subset(c["qcodes"], c["qoff"], qs)) for s, qs in dist.local_blocks(plan, r)]
                for r in range(k)}
        outs = {(r, s): torch.empty((len(qo) - 1, len(sh[s])), dtype=torch.int32, device="cuda")
                for r in range(k) for s, qc, qo in jobs[r]}
        for rep in range(2):            # first pass warms up
            times = []
            for r in range(k):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record()
                for s, qc, qo in jobs[r]:
                    h.search(qc, qo, dbs[s], sw.blosum62(), 10, 2, out=outs[(r, s)])
                e1.record()
                torch.cuda.synchronize()
                times.append(e0.elapsed_time(e1) / 1e3)
    measured = max(times)
    assert abs(plan.makespan - measured) <= 0.10 * measured, (plan.makespan, times)
