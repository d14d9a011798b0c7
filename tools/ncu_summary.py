"""Summarise ncu captures for profiles/ (run here, no GPU needed).

  python tools/ncu_summary.py full  <report.ncu-rep> <out.json>   # --set full capture of one kernel
  python tools/ncu_summary.py launches <launches.csv> <out.json>  # gpu__time_duration launch list

The full summary keeps the evidence the roofline needs: duration, ALU / FMA
pipe utilisation, issue activity, occupancy, DRAM bytes (traffic), stall
reasons and the SASS opcode mix of the DPX cell update.
"""
import csv
import io
import json
import subprocess
import sys
from collections import defaultdict

KEYS = [
    "gpu__time_duration.sum", "launch__grid_size", "launch__block_size", "launch__registers_per_thread",
    "launch__occupancy_limit_registers", "launch__occupancy_limit_shared_mem",
    "sm__pipe_alu_cycles_active.avg.pct_of_peak_sustained_active",
    "sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active",
    "sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active",
    "sm__pipe_fmaheavy_cycles_active.avg.pct_of_peak_sustained_elapsed",
    "smsp__issue_active.avg.pct_of_peak_sustained_active",
    "sm__warps_active.avg.pct_of_peak_sustained_active",
    "smsp__thread_inst_executed_per_inst_executed.ratio",
    "smsp__inst_executed.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
    "dram__bytes.sum.per_second", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum",
    "sm__cycles_elapsed.avg", "smsp__cycles_active.avg",
]


def raw(rep):
    out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    hdr, units = rows[0], rows[1]
    return [(dict(zip(hdr, r)), dict(zip(hdr, units))) for r in rows[2:]]


def full(rep, dst):
    res = []
    for d, u in raw(rep):
        e = {"kernel": d.get("Kernel Name"), "metrics": {}, "stalls_per_issue": {}}
        for k in KEYS:
            if k in d:
                e["metrics"][k] = {"value": d[k], "unit": u.get(k, "")}
        for k, v in d.items():
            if k.startswith("smsp__average_warps_issue_stalled_") and k.endswith("_per_issue_active.ratio"):
                try:
                    if float(v) >= 0.02:
                        e["stalls_per_issue"][k[len("smsp__average_warps_issue_stalled_"):-len("_per_issue_active.ratio")]] = float(v)
                except ValueError:
                    pass
        res.append(e)
    # SASS opcode mix (executed) from the source page
    out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                         capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    mix = defaultdict(int)
    for i, r in enumerate(rows):
        if len(r) > 5 and r[0] == "Address":
            hdr = r
            isrc, iex = hdr.index("Source"), hdr.index("Instructions Executed")
            for rr in rows[i + 1:]:
                if len(rr) <= iex or not rr[iex].isdigit():
                    continue
                op = rr[isrc].strip().split()
                if not op:
                    continue
                o = op[1] if op[0].startswith("@") and len(op) > 1 else op[0]
                mix[o.rstrip(";")] += int(rr[iex])
            break
    if res:
        tot = sum(mix.values()) or 1
        top = sorted(mix.items(), key=lambda kv: -kv[1])[:25]
        res[0]["sass_executed_mix"] = {k: {"warp_instr": v, "frac": round(v / tot, 4)} for k, v in top}
    json.dump(res, open(dst, "w"), indent=1)


def launches(src, dst):
    rows = [r for r in csv.reader(open(src)) if r]
    start = next(i for i, r in enumerate(rows) if "Kernel Name" in r)
    hdr = rows[start]
    ik, iv, imn = hdr.index("Kernel Name"), hdr.index("Metric Value"), hdr.index("Metric Name")
    per = defaultdict(lambda: [0, 0.0])
    total = 0.0
    for r in rows[start + 1:]:
        if len(r) <= iv or r[imn] != "gpu__time_duration.sum":
            continue
        v = float(r[iv].replace(",", ""))
        name = r[ik].split("(")[0]
        per[name][0] += 1
        per[name][1] += v
        total += v
    out = {"total_ns": total, "kernels": {k: {"launches": n, "ns": t, "share": round(t / total, 4) if total else 0}
                                          for k, (n, t) in sorted(per.items(), key=lambda kv: -kv[1][1])}}
    json.dump(out, open(dst, "w"), indent=1)


if __name__ == "__main__":
    {"full": full, "launches": launches}[sys.argv[1]](sys.argv[2], sys.argv[3])
