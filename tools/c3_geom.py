"""Tuning probe (GPU): GCUPS of a whole BASELINE workload (default c3) per forced
(G, R) geometry, DB loaded once.  Env: WL, GEOMS="4,16;4,24;8,16", OPTS="k=v,...".
One JSON line per geometry.  Not part of the product path."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import swgen  # noqa: E402
import paper_conf_icpp_kedad_sidhoummmmt14_b200 as sw  # noqa: E402

c = swgen.make_config(os.environ.get("WL", "c3"))
h = sw.Handle(0, timing=True)
for kv in filter(None, os.environ.get("OPTS", "").split(",")):
    h.set_option(kv.split("=")[0], int(kv.split("=")[1]))
db = h.load_db(c["dcodes"], c["doff"])
S = sw.blosum62()
out = torch.empty((len(c["qoff"]) - 1, db.n_seqs), dtype=torch.int32, device="cuda")
for g in os.environ.get("GEOMS", "0,0;4,16;4,20;4,24;8,16;8,24").split(";"):
    G, R = (int(x) for x in g.split(","))
    h.set_option("force_G", G)
    h.set_option("force_R", R)
    h.search(c["qcodes"], c["qoff"], db, S, 10, 2, out=out)
    torch.cuda.synchronize()
    ms, cells = [], 0
    for _ in range(2):
        h.search(c["qcodes"], c["qoff"], db, S, 10, 2, out=out)
        st = h.last_stats()
        ms.append(st["search_ms"])
        cells = st["cells"]
    print(json.dumps({"G": G, "R": R, "used": [st["last_G"], st["last_R"]], "ms": min(ms),
                      "GCUPS": round(cells / min(ms) / 1e6, 1), "computed/real": round(st["cells_computed"] / cells, 4)}),
          flush=True)
