"""GPU parity: the CUDA path (through the C ABI) vs the CPU oracle, bit-exact.

Inputs are seeded and synthetic (swgen).  Sizes span several strips, lane
groups and chunks with ragged tails; edge cases cover empty sequences, length
1..5, strip boundaries, every kernel geometry, forced and real int16 overflow.
"""
import numpy as np
import pytest

import oracle
import swgen
from oracle.blosum62 import blosum62 as oracle_b62

pytestmark = pytest.mark.gpu

B62_ORACLE = oracle_b62()


def _pkg():
    import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw
    return sw


def gpu_scores(qc, qo, dc, do, S=None, gs=10, ge=2, alpha=24, opts=None, device_out=False):
    sw = _pkg()
    S = sw.blosum62() if S is None else S
    with sw.Handle(0) as h:
        for k, v in (opts or {}).items():
            h.set_option(k, v)
        db = h.load_db(dc, do, alphabet_size=alpha)
        if device_out:
            import torch
            out = h.search(qc, qo, db, S, gs, ge)
            torch.cuda.synchronize()
            return out.cpu().numpy()
        out = np.zeros((len(qo) - 1, len(do) - 1), dtype=np.int32)
        return h.search(qc, qo, db, S, gs, ge, out=out)


def oracle_scores(qc, qo, dc, do, S=None, gs=10, ge=2, procs=8):
    S = B62_ORACLE if S is None else S
    return oracle.gotoh_search(qc, qo, dc, do, S, gs, ge, procs=procs)


def _seqs(lengths, rng, alpha=20):
    lens = np.asarray(lengths, dtype=np.int64)
    off = np.zeros(len(lens) + 1, dtype=np.int64)
    np.cumsum(lens, out=off[1:])
    return rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8), off


def test_matrix_tables_agree():
    sw = _pkg()
    np.testing.assert_array_equal(sw.blosum62().astype(np.int32), B62_ORACLE)


def test_small_random_edges():
    rng = np.random.default_rng(11)
    dl = [0, 1, 2, 3, 4, 5, 7, 8, 31, 32, 33, 63, 64, 65, 127, 128, 129, 255, 256, 257, 300, 511, 512, 513, 0]
    dl += list(rng.integers(1, 700, size=300))
    dc, do = _seqs(dl, rng, alpha=24)
    ql = [1, 2, 7, 8, 9, 31, 32, 33, 64, 100, 255, 256, 257, 500, 767, 768, 769, 1025]
    qc, qo = _seqs(ql, rng, alpha=24)
    np.testing.assert_array_equal(gpu_scores(qc, qo, dc, do), oracle_scores(qc, qo, dc, do))


@pytest.mark.parametrize("G", [4, 8, 16, 32])
@pytest.mark.parametrize("R", [8, 12, 16, 20, 24, 28, 32])
def test_every_geometry(G, R):
    rng = np.random.default_rng(1000 + 37 * G + R)
    dl = list(rng.integers(1, 300, size=90)) + [0, 1, 3, 5]
    dc, do = _seqs(dl, rng)
    # one query spanning 1 strip exactly, one ragged multi-strip
    ql = [G * R, 2 * G * R + 3, 5]
    qc, qo = _seqs(ql, rng)
    got = gpu_scores(qc, qo, dc, do, opts={"force_G": G, "force_R": R})
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


def test_config_c1_full():
    c = swgen.make_config("c1")
    got = gpu_scores(c["qcodes"], c["qoff"], c["dcodes"], c["doff"])
    ref = oracle_scores(c["qcodes"], c["qoff"], c["dcodes"], c["doff"])
    np.testing.assert_array_equal(got, ref)
    assert got.max() > 300  # planted homologs score high


def test_device_output_and_gap_params():
    rng = np.random.default_rng(12)
    dc, do = _seqs(rng.integers(1, 400, size=200), rng)
    qc, qo = _seqs([150, 333], rng)
    for gs, ge in ((10, 2), (0, 1), (11, 1), (5, 5), (0, 0)):
        got = gpu_scores(qc, qo, dc, do, gs=gs, ge=ge, device_out=True)
        np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do, gs=gs, ge=ge))


def test_asymmetric_matrix_small_alphabet():
    rng = np.random.default_rng(13)
    A = 5
    S = rng.integers(-5, 9, size=(A, A)).astype(np.int8)
    dc, do = _seqs(rng.integers(1, 200, size=150), rng, alpha=A)
    qc, qo = _seqs([77, 260], rng, alpha=A)
    got = gpu_scores(qc, qo, dc, do, S=S, gs=3, ge=1, alpha=A)
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do, S=S.astype(np.int32), gs=3, ge=1))


@pytest.mark.parametrize("rows", [0, 8])
def test_forced_overflow_rescore(rows):
    """A tiny threshold sends most pairs through the int32 re-score path (4 rows per
    lane, the automatic choice here, and 8, the choice for queries of >= 2^11 strips)."""
    rng = np.random.default_rng(14)
    dc, do = _seqs(rng.integers(1, 500, size=120), rng)
    qc, qo = _seqs([200, 900], rng)
    sw = _pkg()
    with sw.Handle(0) as h:
        h.set_option("overflow_threshold", 40)
        h.set_option("rescore_rows", rows)
        db = h.load_db(dc, do)
        out = np.zeros((2, 120), dtype=np.int32)
        h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
        st = h.last_stats()
    np.testing.assert_array_equal(out, oracle_scores(qc, qo, dc, do))
    assert st["n_overflow"] > 0


def test_real_int16_overflow():
    """Self-hits of W-rich sequences longer than 32767/11 really wrap int16."""
    rng = np.random.default_rng(15)
    W = 17  # 'W' in NCBI order
    q = np.full(3200, W, dtype=np.uint8)
    q[rng.integers(0, 3200, 40)] = rng.integers(0, 20, 40)
    mut = q.copy()
    mut[rng.integers(0, 3200, 100)] = rng.integers(0, 20, 100)
    dl_other = list(rng.integers(1, 300, size=50))
    others, oo = _seqs(dl_other, rng)
    parts = [q, mut, others]
    dc = np.concatenate(parts)
    do = np.concatenate([[0, len(q), len(q) + len(mut)], len(q) + len(mut) + oo[1:]]).astype(np.int64)
    qc, qo = q.copy(), np.array([0, len(q)], dtype=np.int64)
    got = gpu_scores(qc, qo, dc, do)
    ref = oracle_scores(qc, qo, dc, do)
    assert ref.max() > 32767
    np.testing.assert_array_equal(got, ref)


def test_empty_cases():
    sw = _pkg()
    rng = np.random.default_rng(16)
    dc, do = _seqs([0, 0, 0], rng)
    qc, qo = _seqs([10, 0], rng)
    np.testing.assert_array_equal(gpu_scores(qc, qo, dc, do), np.zeros((2, 3), np.int32))
    dc, do = _seqs([5, 9], rng)
    qc, qo = _seqs([], rng)
    assert gpu_scores(qc, qo, dc, do).shape == (0, 2)


def test_errors():
    sw = _pkg()
    rng = np.random.default_rng(17)
    dc, do = _seqs([5, 9], rng)
    with sw.Handle(0) as h:
        bad = dc.copy()
        bad[0] = 24
        with pytest.raises(sw.SWError):
            h.load_db(bad, do, alphabet_size=24)
        with pytest.raises(sw.SWError):
            h.load_db(dc, do, alphabet_size=33)
        db = h.load_db(dc, do)
        qc, qo = _seqs([4], rng)
        out = np.zeros((1, 2), np.int32)
        with pytest.raises(sw.SWError):
            h.search(qc, qo, db, sw.blosum62(), -1, 2, out=out)
        with pytest.raises(sw.SWError):
            h.search(np.array([30, 1, 2, 3], np.uint8), qo, db, sw.blosum62(), 10, 2, out=out)


@pytest.mark.parametrize("name", ["c2", "c3"])
def test_swissprot_scale_sampled(name):
    """BASELINE configs 2/3 at full size on the GPU; the oracle checks a seeded
    sample of DB sequences (plus every planted homolog and the top hits)."""
    c = swgen.make_config(name)
    got = gpu_scores(c["qcodes"], c["qoff"], c["dcodes"], c["doff"])
    N = len(c["doff"]) - 1
    rng = np.random.default_rng(99)
    sample = set(rng.choice(N, size=300 if name == "c3" else 2000, replace=False).tolist())
    sample |= {p[0] for p in c["plants"]}
    sample |= set(np.argsort(got.max(axis=0))[-20:].tolist())
    idx = np.array(sorted(sample), dtype=np.int64)
    lens = c["doff"][idx + 1] - c["doff"][idx]
    sub_off = np.zeros(len(idx) + 1, dtype=np.int64)
    np.cumsum(lens, out=sub_off[1:])
    sub = np.concatenate([c["dcodes"][c["doff"][i]:c["doff"][i + 1]] for i in idx])
    ref = oracle_scores(c["qcodes"], c["qoff"], sub, sub_off, procs=16)
    np.testing.assert_array_equal(got[:, idx], ref)


def test_intra_task_mode_forced():
    """t_long small: most pairs go through the chained-warps (intra-task) mode;
    queries span 1 strip, 2 strips, and more strips than one CTA's warps (the
    pair is then split into superstrips chained across CTAs)."""
    rng = np.random.default_rng(21)
    dl = list(rng.integers(1, 700, size=70)) + [0, 1, 65, 66, 67, 68]
    dc, do = _seqs(dl, rng)
    ql = [1, 100, 256, 257, 600, 2400, 4100, 13000]   # 13000 rows: the pair is split over 2 CTAs
    qc, qo = _seqs(ql, rng)
    got = gpu_scores(qc, qo, dc, do, opts={"t_long": 64})
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


@pytest.mark.parametrize("pairs", [0, 1])
@pytest.mark.parametrize("G,R", [(4, 24), (8, 24), (16, 12)])
def test_profile_without_bank_copies(G, R, pairs):
    """Option bank_copy 0: one shared-memory copy of the strip profile, unpadded
    letter rows (the layout the bank-spread copies replace)."""
    rng = np.random.default_rng(91 + G + R + pairs)
    dc, do = _seqs(list(rng.integers(1, 400, size=100)) + [0, 2], rng)
    qc, qo = _seqs([2 * G * R + 5, 40, G * R], rng)
    opts = {"bank_copy": 0, "query_pairs": pairs, "force_G": G, "force_R": R}
    got = gpu_scores(qc, qo, dc, do, opts=opts)
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


def test_long_db_sequences():
    rng = np.random.default_rng(22)
    dl = list(rng.integers(3001, 6000, size=24)) + list(rng.integers(1, 400, size=60))
    dc, do = _seqs(dl, rng)
    qc, qo = _seqs([567, 2600, 77], rng)
    got = gpu_scores(qc, qo, dc, do)
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do, procs=16))


def test_config_c4_sampled():
    """BASELINE config 4 (queries 2,000-35,000 vs 1,500 long sequences) in full on
    the GPU; the oracle checks a seeded sample plus every planted long homolog."""
    c = swgen.make_config("c4")
    got = gpu_scores(c["qcodes"], c["qoff"], c["dcodes"], c["doff"])
    N = len(c["doff"]) - 1
    rng = np.random.default_rng(23)
    sample = set(rng.choice(N, size=6, replace=False).tolist()) | {p[0] for p in c["plants"]}
    idx = np.array(sorted(sample), dtype=np.int64)
    lens = c["doff"][idx + 1] - c["doff"][idx]
    sub_off = np.zeros(len(idx) + 1, dtype=np.int64)
    np.cumsum(lens, out=sub_off[1:])
    sub = np.concatenate([c["dcodes"][c["doff"][i]:c["doff"][i + 1]] for i in idx])
    ref = oracle_scores(c["qcodes"], c["qoff"], sub, sub_off, procs=16)
    assert ref.max() > 32767  # planted self-hits of >= 6.4k queries really overflow int16
    np.testing.assert_array_equal(got[:, idx], ref)


@pytest.mark.parametrize("pairs", [0, 1])
def test_query_pairing_modes(pairs):
    """Two queries per register (mode 1) and one (mode 0), odd query counts,
    very unequal pair lengths (the shorter query padded with PAD rows)."""
    rng = np.random.default_rng(31 + pairs)
    dc, do = _seqs(list(rng.integers(1, 600, size=150)) + [0, 1, 2, 3], rng)
    qc, qo = _seqs([700, 31, 256, 255, 1, 90, 400], rng)
    got = gpu_scores(qc, qo, dc, do, opts={"query_pairs": pairs})
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


@pytest.mark.parametrize("pack", [0, 1])
@pytest.mark.parametrize("thr", [0, 40])
def test_query_packing(pack, thr):
    """Mode-1 slots whose shorter half carries several queries laid end to end on
    strip boundaries (a new query starts from a zero boundary row; each query's
    score is emitted at its last strip).  thr > 0 forces the int32 re-score of
    packed queries' pairs (the flag must name the right query)."""
    rng = np.random.default_rng(41 + pack + thr)
    dc, do = _seqs(list(rng.integers(1, 500, size=120)) + [0, 1, 4], rng)
    # strips at G*R = 96: 1900 -> 20, 1100 -> 12, 500 -> 6, 190 -> 2, ...
    ql = [1900, 1100, 500, 190, 96, 97, 5, 1, 800, 380, 33]
    qc, qo = _seqs(ql, rng)
    opts = {"pack_queries": pack, "force_G": 4, "force_R": 24}
    if thr:
        opts["overflow_threshold"] = thr
    got = gpu_scores(qc, qo, dc, do, opts=opts)
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


@pytest.mark.parametrize("skew", [0, 1])
@pytest.mark.parametrize("G,R", [(8, 24), (8, 8), (16, 24), (16, 8), (8, 12), (4, 16), (8, 16)])
def test_single_query_profile_copies(G, R, skew):
    """Single-query mode (two DB sequences per register) with the bank-skewed
    profile copies (option bank_skew, one copy per lane group of a shared-memory
    phase at a searched 4-byte skew) and the linear layout; multi-strip queries."""
    rng = np.random.default_rng(71 + G * 3 + R + skew)
    dc, do = _seqs(list(rng.integers(1, 350, size=120)) + [0, 1, 3], rng)
    qc, qo = _seqs([3 * G * R + 7, G * R, 17], rng)
    opts = {"bank_skew": skew, "query_pairs": 0, "force_G": G, "force_R": R}
    got = gpu_scores(qc, qo, dc, do, opts=opts)
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


@pytest.mark.parametrize("name", ["t5hom", "t5het"])
def test_table5_query_sets_sampled(name):
    """PAPER.md Table V query sets (40 homogeneous 4,500-5,000 aa / heterogeneous
    4-35,213 aa queries) against the Swiss-Prot-sized DB, on the GPU in full; the
    oracle checks a seeded sample of DB sequences plus planted homologs and top hits."""
    c = swgen.make_config(name)
    got = gpu_scores(c["qcodes"], c["qoff"], c["dcodes"], c["doff"])
    N = len(c["doff"]) - 1
    rng = np.random.default_rng(57)
    sample = set(rng.choice(N, size=40, replace=False).tolist())
    sample |= {p[0] for p in c["plants"][::4]}
    sample |= set(np.argsort(got.max(axis=0))[-5:].tolist())
    idx = np.array(sorted(sample), dtype=np.int64)
    lens = c["doff"][idx + 1] - c["doff"][idx]
    sub_off = np.zeros(len(idx) + 1, dtype=np.int64)
    np.cumsum(lens, out=sub_off[1:])
    sub = np.concatenate([c["dcodes"][c["doff"][i]:c["doff"][i + 1]] for i in idx])
    ref = oracle_scores(c["qcodes"], c["qoff"], sub, sub_off, procs=16)
    np.testing.assert_array_equal(got[:, idx], ref)


@pytest.mark.parametrize("gs,ge", [(0, 2), (5, 2)])
def test_nucleotide_mode(gs, ge):
    """DNA over ACGT(N), ma/mi scoring
    (L127-133), linear gap of Eq. (1) as Gs = 0, Ge = -g (L159-165), and the
    affine model, on the same kernels (alphabet 5) vs the oracle; includes the
    Fig. 1 pair (L137-143), whose local optimum is 5."""
    sw = _pkg()
    rng = np.random.default_rng(44 + gs)
    S = sw.nucleotide_matrix(1, -1)
    q = [sw.encode_nucleotide("ACTTGTCCG"), rng.integers(0, 5, size=700).astype(np.uint8),
         rng.integers(0, 4, size=97).astype(np.uint8)]
    qo = np.zeros(4, dtype=np.int64)
    np.cumsum([len(x) for x in q], out=qo[1:])
    dl = [8] + list(rng.integers(1, 1500, size=200)) + [0, 3]
    dc, do = _seqs(dl, rng, alpha=4)
    dc[:8] = sw.encode_nucleotide("ATTGTCAG")
    qc = np.concatenate(q)
    got = gpu_scores(qc, qo, dc, do, S=S, gs=gs, ge=ge, alpha=5)
    ref = oracle_scores(qc, qo, dc, do, S=S.astype(np.int32), gs=gs, ge=ge)
    np.testing.assert_array_equal(got, ref)
    if gs == 0:
        assert got[0, 0] == 5


def test_hybrid_cpu_gpu_search():
    """Hybrid SWDUAL: tasks split between the GPU and 3 host
    PEs by the dual approximation; the assembled matrix equals the oracle's."""
    sw = _pkg()
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    c = swgen.make_config("c1", n_db=900)
    qc, qo = swgen.make_queries(12, [144, 375, 60, 1000])
    with sw.Handle(0) as h:
        hdb = dist.HybridDB(h, c["dcodes"], c["doff"], n_shards=6)
        got, info = hdb.search(qc, qo, sw.blosum62(), 10, 2, n_cpus=3, gpu_rate=2e10, cpu_rate=1e10)
        plan_dp = hdb.plan(np.diff(qo), 3, 2e10, 1e10, variant="dp")
        got_dp, _ = hdb.search(qc, qo, sw.blosum62(), 10, 2, plan=plan_dp)
    plan = info["plan"]
    assert (plan.pe < 3).any() and (plan.pe == 3).any()
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, c["dcodes"], c["doff"]))
    np.testing.assert_array_equal(got_dp, got)


def test_length_limits():
    """Sequences beyond the kernels' counter encoding are refused, not mis-scored."""
    sw = _pkg()
    big = np.zeros((1 << 20), dtype=np.uint8)
    with sw.Handle(0) as h:
        with pytest.raises(sw.SWError) as e:
            h.load_db(big, np.array([0, len(big)], dtype=np.int64))
        assert e.value.code == sw._lib.SW_EUNSUPPORTED
        db = h.load_db(big[:100], np.array([0, 100], dtype=np.int64))
        q = np.zeros((1 << 19) + 1, dtype=np.uint8)
        with pytest.raises(sw.SWError) as e:
            h.search(q, np.array([0, len(q)], dtype=np.int64), db, sw.blosum62(), 10, 2,
                     out=np.zeros((1, 1), dtype=np.int32))
        assert e.value.code == sw._lib.SW_EUNSUPPORTED


def test_mapped_db_writes_into_shared_matrix():
    """sw_load_db_mapped (SURVEY 8(e) fusion): shards loaded with their caller
    columns write straight into one [Q][N] device matrix, leaving the other
    shards' columns untouched (sentinels survive until their own shard runs)."""
    import torch
    sw = _pkg()
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    c = swgen.make_config("c1", n_db=700)
    dc, do = c["dcodes"].copy(), c["doff"].copy()
    lens = np.diff(do)
    lens[5] = 0                                   # an empty sequence: its column must be zeroed
    do = np.zeros(len(lens) + 1, dtype=np.int64)
    np.cumsum(lens, out=do[1:])
    dc = np.concatenate([c["dcodes"][c["doff"][i]:c["doff"][i] + lens[i]] for i in range(len(lens))])
    qc, qo = swgen.make_queries(21, [300, 144, 700])
    N = len(lens)
    shards = dist.shard_cut(do, 3)
    with sw.Handle(0) as h:
        full = torch.full((3, N), -7, dtype=torch.int32, device="cuda")
        dbs = [h.load_db(*dist.subset(dc, do, idx), out_index=idx, out_n=N) for idx in shards]
        h.search(qc, qo, dbs[0], sw.blosum62(), 10, 2, out=full)
        torch.cuda.synchronize()
        part = full.cpu().numpy()
        others = np.setdiff1d(np.arange(N), shards[0])
        assert (part[:, others] == -7).all()
        for db in dbs[1:]:
            h.search(qc[:0], qo[:1], db, sw.blosum62(), 10, 2, out=full[:0])   # no queries: writes nothing
        h.search(qc[qo[1]:], qo[1:] - qo[1], dbs[1], sw.blosum62(), 10, 2, out=full[1:])   # rows 1..2 only
        h.search(qc, qo, dbs[2], sw.blosum62(), 10, 2, out=full)
        h.search(qc[:qo[1]], qo[:2], dbs[1], sw.blosum62(), 10, 2, out=full[:1])          # row 0
        torch.cuda.synchronize()
        got = full.cpu().numpy()
        with pytest.raises(sw.SWError):   # host output is refused for a mapped DB
            h.search(qc, qo, dbs[0], sw.blosum62(), 10, 2, out=np.zeros((3, N), dtype=np.int32))
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


def test_mapped_db_resets_its_columns():
    """A mapped DB writes every one of its columns in every query row: a stale
    positive value (reused buffer) never survives, not for a long pair split
    over several CTAs (a > 13k-row query) nor for an empty query's zero row."""
    import torch
    sw = _pkg()
    from paper_conf_icpp_kedad_sidhoummmmt14_b200 import dist
    rng = np.random.default_rng(77)
    dl = list(rng.integers(3001, 4500, size=6)) + list(rng.integers(1, 400, size=40)) + [0]
    dc, do = _seqs(dl, rng)
    qc, qo = _seqs([13500, 0, 300], rng)
    N = len(dl)
    shards = dist.shard_cut(do, 2)
    with sw.Handle(0) as h:
        full = torch.full((3, N), 30000, dtype=torch.int32, device="cuda")   # stale, above every true score
        for idx in shards:
            db = h.load_db(*dist.subset(dc, do, idx), out_index=idx, out_n=N)
            h.search(qc, qo, db, sw.blosum62(), 10, 2, out=full)
        torch.cuda.synchronize()
        got = full.cpu().numpy()
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


def test_searches_on_two_streams_share_the_handle():
    """Back-to-back searches of one handle on two streams, no host sync between
    them (the second waits for the first on the device): both exact."""
    import torch
    sw = _pkg()
    rng = np.random.default_rng(78)
    dc, do = _seqs(list(rng.integers(1, 600, size=300)), rng)
    qa, qao = _seqs([700, 150, 3300], rng)
    qb, qbo = _seqs([90, 2000], rng)
    s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
    with sw.Handle(0) as h:
        h.set_option("overflow_threshold", 60)      # both searches also run the re-score kernel
        db = h.load_db(dc, do)
        oa = torch.empty((3, 300), dtype=torch.int32, device="cuda")
        ob = torch.empty((2, 300), dtype=torch.int32, device="cuda")
        for _ in range(3):
            h.search(qa, qao, db, sw.blosum62(), 10, 2, out=oa, stream=s1)
            h.search(qb, qbo, db, sw.blosum62(), 10, 2, out=ob, stream=s2)
        torch.cuda.synchronize()
        ga, gb = oa.cpu().numpy(), ob.cpu().numpy()
    np.testing.assert_array_equal(ga, oracle_scores(qa, qao, dc, do))
    np.testing.assert_array_equal(gb, oracle_scores(qb, qbo, dc, do))


def test_overflow_threshold_is_clamped():
    """A forced threshold above 32767 - S_max is lowered to it, so real int16
    overflow is still flagged and re-scored exactly."""
    rng = np.random.default_rng(79)
    W = 17
    q = np.full(3300, W, dtype=np.uint8)
    q[rng.integers(0, 3300, 30)] = rng.integers(0, 20, 30)
    dc = np.concatenate([q, rng.integers(0, 20, 500).astype(np.uint8)])
    do = np.array([0, len(q), len(q) + 500], dtype=np.int64)
    got = gpu_scores(q, np.array([0, len(q)], np.int64), dc, do, opts={"overflow_threshold": 40000})
    ref = oracle_scores(q, np.array([0, len(q)], np.int64), dc, do)
    assert ref.max() > 32767
    np.testing.assert_array_equal(got, ref)


@pytest.mark.parametrize("cg", [0, 1])
@pytest.mark.parametrize("pairs", [0, 1])
def test_constant_gap_kernels(cg, pairs):
    """Gs = 10, Ge = 2 searches run the constant-gap instantiations (penalties as
    immediates) unless option const_gaps is 0; both give the oracle's scores,
    multi-strip queries included."""
    rng = np.random.default_rng(95 + 2 * cg + pairs)
    dc, do = _seqs(list(rng.integers(1, 500, size=150)) + [0, 1, 3], rng)
    qc, qo = _seqs([700, 129, 64, 3100, 2], rng)
    got = gpu_scores(qc, qo, dc, do, opts={"const_gaps": cg, "query_pairs": pairs})
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


NIB_GEOMS = [(4, 16), (4, 24), (4, 32), (8, 16), (8, 24), (16, 12), (16, 24), (32, 8), (32, 16)]


@pytest.mark.parametrize("G,R", NIB_GEOMS)
@pytest.mark.parametrize("pairs", [0, 1])
def test_nibble_stream_geometries(G, R, pairs):
    """alphabets <= 15 (DNA/RNA, alphabet 5 with N) are packed 4 bits
    per residue (two codes per byte of the pair stream, half the DB bytes); every
    4-bit instantiation, both query modes, multi-strip queries and PAD columns."""
    sw = _pkg()
    rng = np.random.default_rng(200 + G * 3 + R + pairs)
    S = sw.nucleotide_matrix(2, -3)
    dc, do = _seqs(list(rng.integers(1, 600, size=130)) + [0, 1, 2, 5], rng, alpha=5)
    qc, qo = _seqs([3 * G * R + 7, G * R, 40, 1, 333], rng, alpha=5)
    got = gpu_scores(qc, qo, dc, do, S=S, gs=5, ge=2, alpha=5,
                     opts={"force_G": G, "force_R": R, "query_pairs": pairs})
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do, S=S.astype(np.int32), gs=5, ge=2))


@pytest.mark.parametrize("opts", [{"t_long": 64}, {"overflow_threshold": 30}, {"nibble": 0}, {}])
def test_nibble_stream_long_rescore_and_off(opts):
    """4-bit streams through the intra-task kernel (forced long pairs, queries of
    1 to 26 strips), the int32 re-score (forced threshold), and the 8-bit layout
    (option nibble 0) for the same nucleotide DB: all equal to the oracle."""
    sw = _pkg()
    rng = np.random.default_rng(210 + len(str(opts)))
    S = sw.nucleotide_matrix(1, -1)
    dc, do = _seqs(list(rng.integers(1, 900, size=80)) + [0, 1, 66, 67], rng, alpha=5)
    qc, qo = _seqs([1, 100, 513, 2400, 4100, 13000], rng, alpha=5)
    got = gpu_scores(qc, qo, dc, do, S=S, gs=0, ge=2, alpha=5, opts=opts)
    np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do, S=S.astype(np.int32), gs=0, ge=2))


@pytest.mark.parametrize("small", [0, 1])
def test_small_search_one_group_ctas(small):
    """Latency-bound single-query searches at G = 32 run one lane group per
    32-thread CTA (option small_ctas); both layouts equal the oracle, including
    multi-strip queries and the longest pair setting the critical path."""
    rng = np.random.default_rng(230 + small)
    dc, do = _seqs(list(rng.integers(1, 700, size=300)) + [2005, 0, 1], rng)
    for ql in ([144], [700], [33]):
        qc, qo = _seqs(ql, rng)
        got = gpu_scores(qc, qo, dc, do, opts={"small_ctas": small})
        np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do))


def test_long_only_search_tall_queries():
    """A search whose pairs are all long (every DB sequence longer than t_long)
    runs the long kernel alone: tall queries chain their strips over the warps
    of one CTA in rounds (the round wrap through global memory); the host packs
    several pairs per item when that leaves fewer warps idle.  Equals the oracle."""
    rng = np.random.default_rng(240)
    dc, do = _seqs(list(rng.integers(70, 900, size=24)) + [3001, 1500], rng)
    # 1,024-row strips (32 lanes x 32 rows): 13 / 35 strips over 8 warps per pair (2 / 5
    # rounds, the round wrap through global memory); 2 strips: 4 pairs of 2 warps; 5 and
    # 10 strips: 8 pairs of 1 warp / 4 pairs of 2 warps (one round-wrap row per pair group)
    for ql in ([13000, 100, 700], [35000, 2000], [5000, 10000, 300]):
        qc, qo = _seqs(ql, rng)
        got = gpu_scores(qc, qo, dc, do, opts={"t_long": 64})
        np.testing.assert_array_equal(got, oracle_scores(qc, qo, dc, do, procs=16))
