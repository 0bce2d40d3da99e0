#!/usr/bin/env python3
"""Code layout of a kernel from ncu source pages: which source lines the cold gaps inside the hot address
span come from (candidates for out-of-line placement; stall_no_inst tracks the hot span).
usage: code_layout.py sass.csv src.csv [window_bytes]"""
import collections
import csv
import sys

sass = list(csv.reader(open(sys.argv[1], errors="replace")))
hdr = next(r for r in sass if r and r[0] == "Address")
ia = hdr.index("Instructions Executed")
cnt = {}
for r in sass:
    if r and r[0].startswith("0x"):
        try:
            cnt[int(r[0], 16)] = float(r[ia] or 0)
        except ValueError:
            pass
src = {}
fname, line = "?", "?"
for r in csv.reader(open(sys.argv[2], errors="replace")):
    if not r:
        continue
    if r[0] == "File Path":
        fname = r[1].split("/")[-1]
        continue
    if r[0] and r[0].isdigit():
        line = "%s:%s" % (fname, r[0])
    if len(r) > 2 and r[2].startswith("0x"):
        src[int(r[2], 16)] = line
base = min(cnt)
tot = sum(cnt.values())
hot = sorted(a for a, c in cnt.items() if c > 1e-4 * tot / len(cnt) * 50)
lo, hi = hot[0], hot[-1]
W = int(sys.argv[3]) if len(sys.argv) > 3 else 1024
print("hot span 0x%x..0x%x (%.1f KB)" % (lo - base, hi - base, (hi - lo) / 1024))
for w0 in range(lo, hi + 1, W):
    addrs = [a for a in range(w0, w0 + W, 16) if a in cnt]
    ex = sum(cnt[a] for a in addrs)
    cold = [a for a in addrs if cnt[a] == 0]
    lines = collections.Counter(src.get(a, "?") for a in cold)
    print("+%6.1fK exec %5.2f%% cold %3d/%3d  %s" % ((w0 - base) / 1024, 100 * ex / tot, len(cold), len(addrs),
          ", ".join("%s(%d)" % kv for kv in lines.most_common(4))))
