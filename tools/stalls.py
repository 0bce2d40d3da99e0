#!/usr/bin/env python3
"""Stall-reason totals (and top source lines per reason) from an ncu source-page CSV
(ncu -i X.ncu-rep --page source --csv --print-source cuda,sass)."""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
hdr = next(r for r in rows if r and r[0] == "Line No")
cols = {h: i for i, h in enumerate(hdr) if h.startswith("stall_") and "(Not" not in h}
tot = {h: 0.0 for h in cols}
per_line = {}
fname = "?"
for r in rows:
    if not r or r[0] in ("Line No", "Function Name"):
        continue
    if r[0] == "File Path":
        fname = r[1].split("/")[-1]
        continue
    if r[0] != "":
        key = "%s:%s %s" % (fname, r[0], r[1][:70])
        for h, i in cols.items():
            try:
                v = float(r[i] or 0)
            except ValueError:
                continue
            tot[h] += v
            per_line.setdefault(h, {}).setdefault(key, 0.0)
            per_line[h][key] += v
s = sum(tot.values())
for h, v in sorted(tot.items(), key=lambda kv: -kv[1]):
    if v / s < 0.01:
        continue
    print("%-24s %5.1f%%" % (h, 100 * v / s))
    for k, x in sorted(per_line[h].items(), key=lambda kv: -kv[1])[:4]:
        print("      %5.1f%%  %s" % (100 * x / s, k))
