"""Summarise `nvcc -Xptxas -v` output (stdin): kernel, registers, spill bytes."""
import re, sys
cur = None
for line in sys.stdin:
    m = re.search(r"Compiling entry function '(\S+)'", line)
    if m: cur = m.group(1); continue
    m = re.search(r"(\d+) bytes stack frame, (\d+) bytes spill stores, (\d+) bytes spill loads", line)
    if m and cur: st = m.groups(); continue
    m = re.search(r"Used (\d+) registers", line)
    if m and cur:
        name = re.sub(r"_ZN6swdual\d+", "", cur)
        print(f"{name[:60]:60s} regs={m.group(1):>4} stack={st[0]} spill_st={st[1]} spill_ld={st[2]}")
        cur = None
