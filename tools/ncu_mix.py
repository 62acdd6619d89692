#!/usr/bin/env python
"""Instruction mix + stall totals of an ncu report's source page (SASS)."""
import csv
import io
import subprocess
import sys
from collections import Counter

rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(out)))
hdr, data = rows[1], rows[2:]
iE = hdr.index("Instructions Executed")
cols = [c for c in hdr if c.startswith("stall_") and "Not Issued" not in c]
tot = Counter()
for r in data:
    for c in cols:
        tot[c] += int(r[hdr.index(c)] or 0)
print("stalls:", ", ".join(f"{k[6:]}={v}" for k, v in tot.most_common(10)))
mix = Counter()
for r in data:
    t = r[1].split()
    op = (t[1] if t and t[0].startswith("@") else t[0]).split(".")[0] if t else "?"
    mix[op] += int(r[iE] or 0)
n = sum(mix.values())
print("warp instructions:", n)
print("  ".join(f"{op} {100 * c / n:.1f}%" for op, c in mix.most_common(22)))
