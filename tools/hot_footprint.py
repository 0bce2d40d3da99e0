#!/usr/bin/env python3
"""Hot-code footprint of a kernel from an ncu SASS source page (ncu -i X --page source --csv
--print-source sass): how many distinct instructions (x16 B) cover 90/99/99.9 % of executed warp
instructions, and the address span they occupy.  Instruction fetch (stall_no_inst) tracks this."""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1], errors="replace")))
hdr = next(r for r in rows if r and r[0] == "Address")
ia = hdr.index("Instructions Executed")
ins = []
for r in rows:
    if not r or not r[0].startswith("0x"):
        continue
    try:
        ins.append((int(r[0], 16), float(r[ia] or 0)))
    except ValueError:
        pass
tot = sum(c for _, c in ins)
print("instructions in kernel: %d (%.1f KB); executed warp-inst: %.3g" % (len(ins), len(ins) * 16 / 1024, tot))
srt = sorted(ins, key=lambda x: -x[1])
for q in (0.9, 0.99, 0.999):
    acc, k = 0.0, 0
    for a, c in srt:
        acc += c
        k += 1
        if acc >= q * tot:
            break
    addrs = sorted(a for a, _ in srt[:k])
    # number of distinct 128-byte lines touched
    lines = len({a // 128 for a in addrs})
    print("%.1f%%: %d instructions (%.1f KB) in %d 128-B lines, span %.1f KB"
          % (100 * q, k, k * 16 / 1024, lines, (addrs[-1] - addrs[0]) / 1024))
