#!/usr/bin/env python
"""Summarise an `ncu --set full` capture and a launch list into profiles/.

usage: python tools/ncu_summary.py <prof.ncu-rep|raw.csv> <launches.csv|-> <tag> <workload-key> [<bench-log>]
Writes profiles/<tag>_ncu_full.txt, profiles/<tag>_launches.csv and merges the per-launch
DRAM bytes into profiles/ncu_traffic.json (read by bench.py for roofline.traffic).  The entry is
keyed by the source-tree hash and launch plan of the captured run, taken from the bench.py JSON
line in <bench-log> (the stdout of the command ncu profiled), so bench.py quotes it only for the
same tree and launch.
"""
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
KEYS = [
    "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum", "dram__bytes.sum.per_second",
    "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
    "lts__t_bytes.sum", "launch__registers_per_thread", "launch__grid_size", "launch__block_size",
    "launch__shared_mem_per_block_dynamic", "sm__warps_active.avg.pct_of_peak_sustained_active",
    "smsp__inst_executed.sum", "l1tex__data_pipe_lsu_wavefronts_mem_shared_op_ld.sum",
    "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum",
    "sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active", "sm__cycles_elapsed.avg.per_second",
    "smsp__pcsamp_warps_issue_stalled_long_scoreboard", "smsp__pcsamp_warps_issue_stalled_barrier",
    "smsp__pcsamp_warps_issue_stalled_wait", "smsp__pcsamp_warps_issue_stalled_short_scoreboard",
]


def raw(rep):
    """The raw metric page: from a report (ncu -i) or from its CSV export (`ncu -i rep --page raw --csv`)."""
    if rep.endswith(".csv"):
        with open(rep) as f:
            out = f.read()
    else:
        out = subprocess.run(["ncu", "-i", rep, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(out)))
    return rows[0], rows[1], rows[2:]


def bench_line(path):
    with open(path) as f:
        for line in f:
            if line.startswith("{"):
                return json.loads(line)
    return None


def main():
    rep, launches, tag, key = sys.argv[1:5]
    bl = bench_line(sys.argv[5]) if len(sys.argv) > 5 else None
    hdr, units, rows = raw(rep)
    lines = [f"# ncu --set full summary: {os.path.basename(rep)} (tag {tag}, workload {key})"]
    per = []
    for r in rows:
        name = r[hdr.index("Kernel Name")] if "Kernel Name" in hdr else "?"
        lines.append(f"\n## {name}")
        d = {}
        for k in KEYS:
            if k in hdr:
                i = hdr.index(k)
                lines.append(f"{k} = {r[i]} {units[i]}")
                d[k] = (r[i], units[i])
        per.append(d)
    prof_dir = os.path.join(ROOT, "profiles")
    with open(os.path.join(prof_dir, f"{tag}_ncu_full.txt"), "w") as f:
        f.write("\n".join(lines) + "\n")

    def to_bytes(v, u):
        v = float(v.replace(",", ""))
        return v * {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12}.get(u, 1)

    if per and bl is not None:
        sys.path.insert(0, ROOT)
        import bench

        d = per[-1]
        rb = to_bytes(*d["dram__bytes_read.sum"])
        wb = to_bytes(*d["dram__bytes_write.sum"])
        path = os.path.join(prof_dir, "ncu_traffic.json")
        allv = json.load(open(path)) if os.path.exists(path) else {}
        allv[key] = {"dram_bytes_per_launch": rb + wb, "dram_read": rb, "dram_write": wb, "tag": tag,
                     "duration": d["gpu__time_duration.sum"][0] + " " + d["gpu__time_duration.sum"][1],
                     "dram_pct_of_peak": float(d["gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed"][0]),
                     "src_hash": bl["launch"]["src_hash"], "plan": bench.plan_key(bl["launch"]["plan"])}
        json.dump(allv, open(path, "w"), indent=1)
    # launch list
    if launches == "-":
        print("\n".join(lines[:40]))
        return
    with open(launches) as f:
        txt = f.read()
    rows = [r for r in csv.reader(io.StringIO(txt[txt.index('"ID"'):]))]
    h = rows[0]
    out = ["kernel,duration_ns"]
    tot = {}
    for r in rows[1:]:
        if r[h.index("Metric Name")] != "gpu__time_duration.sum":
            continue
        nm = r[h.index("Kernel Name")].split("(")[0]
        ns = float(r[h.index("Metric Value")].replace(",", ""))
        out.append(f"\"{nm}\",{ns:.0f}")
        tot[nm] = tot.get(nm, 0) + ns
    s = sum(tot.values())
    out.append("")
    out.append("# share of summed device time per kernel (cold-cache, serialised)")
    for nm, ns in sorted(tot.items(), key=lambda kv: -kv[1]):
        out.append(f"# {nm}: {100 * ns / s:.1f}%")
    with open(os.path.join(prof_dir, f"{tag}_launches.csv"), "w") as f:
        f.write("\n".join(out) + "\n")
    print("\n".join(lines[:40]))


if __name__ == "__main__":
    main()
