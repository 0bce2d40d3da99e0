"""Hot instructions of an ncu source-page CSV (--page source --csv --print-source sass): top stall sites,
CCTL/fence counts.  python tools/sass_hot.py <sass.csv> [stall_column] [n]"""
import csv, sys
rows = list(csv.reader(open(sys.argv[1])))
h = rows[1]; data = rows[2:]
col = sys.argv[2] if len(sys.argv) > 2 else "stall_long_sb"
n = int(sys.argv[3]) if len(sys.argv) > 3 else 20
ai, si, ti, ei = h.index("Address"), h.index("Source"), h.index("Warp Stall Sampling (All Samples)"), h.index("Instructions Executed")
ci = h.index(col)
f = lambda x: float(x) if x not in ("", None) else 0.0
tot = sum(f(r[ti]) for r in data)
print("samples", tot, col, sum(f(r[ci]) for r in data))
for name in [c for c in h if c.startswith("stall_") and "Not Issued" not in c]:
    v = sum(f(r[h.index(name)]) for r in data)
    if v > 0.01 * tot:
        print("  %-24s %5.1f%%" % (name, 100 * v / tot))
for r in sorted(data, key=lambda r: -f(r[ci]))[:n]:
    print(r[ai][-6:], "%7.0f %7.0f %12.0f" % (f(r[ci]), f(r[ti]), f(r[ei])), r[si].strip()[:70])
for r in data:
    if ("CCTL" in r[si] or "MEMBAR" in r[si]) and f(r[ei]) > 1e5:
        print("fence", r[ai][-6:], r[si].strip()[:40], r[ei])
