"""Aggregate `ncu --page source --csv --print-source sass` by opcode and by hot
basic region: python tools/ncu_src_ops.py a.csv [b.csv]"""
import csv, sys, collections, re
def load(p):
    rows = list(csv.reader(open(p)))
    hdr = rows[1]
    ia, isrc, iex, ism = hdr.index("Address"), hdr.index("Source"), hdr.index("Instructions Executed"), hdr.index("Warp Stall Sampling (All Samples)")
    ops, samp = collections.Counter(), collections.Counter()
    tot = 0
    for r in rows[2:]:
        if len(r) <= iex: continue
        src = re.sub(r"^@!?U?P\w+\s+", "", r[isrc].strip())
        op = src.split()[0] if src else "?"
        n = int(r[iex] or 0); s = int(r[ism] or 0)
        ops[op] += n; samp[op] += s; tot += n
    return ops, samp, tot
res = [load(p) for p in sys.argv[1:]]
keys = sorted(set().union(*[r[0] for r in res]), key=lambda k: -res[0][0].get(k, 0))
print("op".ljust(26), *[f"{p[-14:]:>16s}" for p in sys.argv[1:]])
for k in keys[:30]:
    print(k.ljust(26), *[f"{r[0].get(k,0):16d}" for r in res], *[f"{r[1].get(k,0):8d}" for r in res])
print("TOTAL".ljust(26), *[f"{r[2]:16d}" for r in res])
