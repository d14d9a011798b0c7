"""Split a cuobjdump -sass listing into basic blocks (by branch targets) and
print, for each block with one of the given opcodes, its address range, size
and opcode histogram.  Usage: python tools/sass_blocks.py file.sass LDS.128"""
import re, sys, collections
lines = open(sys.argv[1]).read().splitlines()
want = sys.argv[2:] or ["LDS.128"]
ins = []
for l in lines:
    m = re.match(r"\s+/\*([0-9a-f]{4,})\*/\s+(.*?);", l)
    if m:
        ins.append((int(m.group(1), 16), m.group(2).strip()))
targets = set()
for a, t in ins:
    m = re.search(r"BRA(?:\.\w+)*\s+(?:\S+,\s*)?0x([0-9a-f]+)", t)
    if m:
        targets.add(int(m.group(1), 16))
blocks, cur = [], []
for a, t in ins:
    if a in targets and cur:
        blocks.append(cur); cur = []
    cur.append((a, t))
    if re.search(r"\bBRA\b|EXIT|RET", t):
        blocks.append(cur); cur = []
if cur: blocks.append(cur)
for b in blocks:
    ops = collections.Counter(re.sub(r"^@!?U?P\w+\s+", "", t).split()[0] for _, t in b)
    if any(w in ops for w in want) and len(b) > 20:
        back = [t for _, t in b if "BRA" in t]
        print(f"{b[0][0]:#07x}-{b[-1][0]:#07x} n={len(b)} {back[-1] if back else ''}")
        print("   ", ", ".join(f"{k}:{v}" for k, v in ops.most_common(16)))
