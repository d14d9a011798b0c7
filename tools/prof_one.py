"""Run a few searches of one query length against the Swiss-Prot-sized DB (for ncu)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402

m = int(os.environ.get("PROF_M", "567") or 567)
reps = int(os.environ.get("PROF_REPS", "2"))
wl = os.environ.get("PROF_WORKLOAD", "c2")
c = swgen.make_config(wl, n_db=int(os.environ["PROF_NDB"]) if os.environ.get("PROF_NDB") else None)
h = sw.Handle(0)
for kv in filter(None, os.environ.get("SWDUAL_OPTS", "").split(",")):
    h.set_option(kv.split("=")[0], int(kv.split("=")[1]))
for k in ("force_G", "force_R"):
    if os.environ.get(k.upper()):
        h.set_option(k, int(os.environ[k.upper()]))
db = h.load_db(c["dcodes"], c["doff"])
if os.environ.get("PROF_M"):
    qc, qo = swgen.make_queries(77, [m])
else:
    qc, qo = c["qcodes"], c["qoff"]
out = torch.empty((len(qo) - 1, db.n_seqs), dtype=torch.int32, device="cuda")
for _ in range(reps):
    h.search(qc, qo, db, sw.blosum62(), 10, 2, out=out)
torch.cuda.synchronize()
print("done", int(out.max()))
