"""Debug: dump the traceback codes of one sw_align pair and diff them against a
direct full-matrix computation of the same codes."""
import sys, os
import numpy as np
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw

def seqs(lengths, rng, alpha):
    lens = np.asarray(lengths, dtype=np.int64); off = np.zeros(len(lens) + 1, dtype=np.int64); np.cumsum(lens, out=off[1:])
    return rng.integers(0, alpha, size=int(off[-1])).astype(np.uint8), off
alpha, gs, ge = 4, 3, 1
rng = np.random.default_rng(100 + 7 * alpha + gs + 3 * ge)
S = rng.integers(-4, 6, size=(alpha, alpha))
ql = [1, 2, 7, 31, 255, 256, 257, 600]; dl = [1, 3, 4, 5, 9, 64, 250, 333, 700, 2]
qc, qo = seqs(ql, rng, alpha); dc, do = seqs(dl, rng, alpha)
qi, di = int(sys.argv[1]), int(sys.argv[2])
os.environ["SWDUAL_ALIGN_DUMP"] = "gpurun_out/trace.bin"
with sw.Handle(0) as h:
    db = h.load_db(dc, do, alphabet_size=alpha)
    got = h.align(qc, qo, db, [(qi, di)], S.astype(np.int8), gs, ge)
print(got[0][:5])
tr = np.fromfile("gpurun_out/trace.bin", dtype=np.uint32)
q = qc[qo[qi]:qo[qi + 1]]; d = dc[do[di]:do[di + 1]]
m, n = len(q), len(d); GsGe = gs + ge
T = ((n + 3) & ~3) + 32
H = np.zeros((m + 1, n + 1), np.int64); E = H.copy(); F = H.copy(); code = H.copy()
for i in range(1, m + 1):
    for j in range(1, n + 1):
        E[i, j] = max(E[i, j - 1] - ge, H[i, j - 1] - GsGe, 0); F[i, j] = max(F[i - 1, j] - ge, H[i - 1, j] - GsGe, 0)
        dg = H[i - 1, j - 1] + S[q[i - 1], d[j - 1]]; hh = max(dg, E[i, j], F[i, j], 0); H[i, j] = hh
        src = 0 if hh == 0 else 1 if hh == dg else 2 if hh == E[i, j] else 3
        code[i, j] = src | (4 if E[i, j] == H[i, j - 1] - GsGe else 0) | (8 if F[i, j] == H[i - 1, j] - GsGe else 0)
nb = 0
for i in range(1, m + 1):
    for j in range(1, n + 1):
        r, c = i - 1, j - 1
        s, ln, rr = r >> 8, (r >> 3) & 31, r & 7
        w = int(tr[(s * T + c + ln) * 32 + ln]); g = (w >> (4 * rr)) & 15
        if g != code[i, j]:
            nb += 1
            if nb < 15: print("cell", i, j, "gpu", g, "ref", code[i, j], "H", H[i, j], "E", E[i, j], "F", F[i, j], "Hup", H[i-1, j], "Hleft", H[i, j-1])
print("mismatching cells", nb, "of", m * n)
