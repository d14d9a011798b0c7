"""Debug helper for sw_align parity: one failing case run three ways."""
import sys, os
import numpy as np
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw

def seqs(lengths, rng, alpha):
    lens = np.asarray(lengths, dtype=np.int64); off = np.zeros(len(lens) + 1, dtype=np.int64); np.cumsum(lens, out=off[1:])
    return rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8), off
alpha, gs, ge = 4, 3, 1
rng = np.random.default_rng(100 + 7 * alpha + gs + 3 * ge)
S = rng.integers(-4, 6, size=(alpha, alpha))
ql = [1, 2, 7, 31, 255, 256, 257, 600]; dl = [1, 3, 4, 5, 9, 64, 250, 333, 700, 2]
qc, qo = seqs(ql, rng, alpha); dc, do = seqs(dl, rng, alpha)
pairs = [(q, d) for q in range(len(ql)) for d in range(len(dl))]
ref = [oracle.gotoh_align(qc[qo[q]:qo[q + 1]], dc[do[d]:do[d + 1]], S.astype(np.int32), gs, ge) for q, d in pairs]
for name, ws, sel in [("all", 2048, range(len(pairs))), ("ws1", 1, range(len(pairs))), ("single27", 2048, [27])]:
    with sw.Handle(0) as h:
        h.set_option("align_workspace_mb", ws)
        db = h.load_db(dc, do, alphabet_size=alpha)
        got = h.align(qc, qo, db, [pairs[k] for k in sel], S.astype(np.int8), gs, ge)
    bad = [(k, pairs[k], got[i][:5], ref[k][:5]) for i, k in enumerate(sel) if tuple(got[i][:5]) != ref[k][:5] or got[i][5] != ref[k][5]]
    print(name, "bad", len(bad), "of", len(sel), bad[:6])
# same-sequence: q vs itself embedded
