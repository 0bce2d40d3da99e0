#!/usr/bin/env python3
"""Summarise ncu output for profiles/: launch-list shares and the key metrics of a --set full capture.

  python tools/ncu_summary.py launches <launches.csv>
  python tools/ncu_summary.py full <prof.ncu-rep> [--json out.json] [--steps S]
"""
from __future__ import annotations

import csv
import io
import json
import subprocess
import sys

KEYS = [
    "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum", "smsp__inst_executed.sum",
    "smsp__thread_inst_executed_per_inst_executed.ratio", "lts__t_sector_hit_rate.pct",
    "l1tex__t_sector_hit_rate.pct", "smsp__issue_active.avg.pct_of_peak_sustained_active",
    "sm__warps_active.avg.pct_of_peak_sustained_active", "launch__registers_per_thread",
    "launch__grid_size", "launch__block_size", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
    "sm__cycles_elapsed.avg.per_second", "smsp__sass_inst_executed_op_global_ld.sum",
    "smsp__sass_inst_executed_op_global_st.sum", "smsp__sass_inst_executed_op_local_ld.sum",
    "smsp__sass_inst_executed_op_shared_ld.sum", "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed",
    "smsp__warp_issue_stalled_long_scoreboard_per_warp_active.pct",
    "smsp__warp_issue_stalled_short_scoreboard_per_warp_active.pct",
    "smsp__warp_issue_stalled_wait_per_warp_active.pct",
    "smsp__warp_issue_stalled_branch_resolving_per_warp_active.pct",
    "smsp__warp_issue_stalled_no_instruction_per_warp_active.pct",
    "smsp__warp_issue_stalled_lg_throttle_per_warp_active.pct",
    "smsp__warp_issue_stalled_mio_throttle_per_warp_active.pct",
    "smsp__warp_issue_stalled_math_pipe_throttle_per_warp_active.pct",
    "smsp__warp_issue_stalled_not_selected_per_warp_active.pct",
    "smsp__warp_issue_stalled_selected_per_warp_active.pct",
    "smsp__warp_issue_stalled_dispatch_stall_per_warp_active.pct",
]


def launches(path):
    rows = list(csv.reader(open(path)))
    hi = next(i for i, r in enumerate(rows) if "Kernel Name" in r)
    h = rows[hi]
    ki, vi = h.index("Kernel Name"), h.index("Metric Value")
    agg = {}
    for r in rows[hi + 1:]:
        if len(r) <= vi:
            continue
        agg.setdefault(r[ki].split("(")[0], []).append(float(r[vi].replace(",", "")))
    tot = sum(sum(v) for v in agg.values())
    out = ["| kernel | launches | total ms | share |", "|---|---|---|---|"]
    for k, v in sorted(agg.items(), key=lambda kv: -sum(kv[1])):
        out.append("| %s | %d | %.3f | %.2f%% |" % (k[:80], len(v), sum(v) / 1e6, 100 * sum(v) / tot))
    return "\n".join(out)


def full(path):
    raw = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True,
                         text=True).stdout
    rows = list(csv.reader(io.StringIO(raw)))
    hdr, units = rows[0], rows[1]
    res = []
    for vals in rows[2:]:
        d = {}
        for k in KEYS:
            if k in hdr:
                i = hdr.index(k)
                d[k] = (vals[i], units[i])
        d["Kernel Name"] = vals[hdr.index("Kernel Name")] if "Kernel Name" in hdr else "?"
        res.append(d)
    return res


def num(s):
    return float(str(s).replace(",", ""))


UNIT = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "ns": 1e-9, "nsecond": 1e-9, "us": 1e-6,
        "usecond": 1e-6, "ms": 1e-3, "msecond": 1e-3, "s": 1.0, "second": 1.0}


def sweep(paths, peak_gbs=6547.5):
    """Per workload and kernel (first launch of each kernel in the capture): the SURVEY §8(d) metrics."""
    out = ["| config | kernel | time ms | DRAM GB | DRAM GB/s | %% of %.0f GB/s | warp eff. | L2 hit | issue active "
           "| warps active | local B |" % peak_gbs, "|---|---|---|---|---|---|---|---|---|---|---|"]
    for path in paths:
        wl = path.rsplit("_", 1)[-1].split(".")[0]
        rows = list(csv.reader(open(path, errors="replace")))
        try:
            hi = next(i for i, r in enumerate(rows) if "Metric Name" in r)
        except StopIteration:
            out.append("| %s | (no data) |" % wl)
            continue
        h = rows[hi]
        ii, ki, mi, ui, vi = (h.index(x) for x in ("ID", "Kernel Name", "Metric Name", "Metric Unit", "Metric Value"))
        per = {}
        for r in rows[hi + 1:]:
            if len(r) <= vi:
                continue
            per.setdefault((r[ki].split("(")[0], r[ii]), {})[r[mi]] = num(r[vi]) * UNIT.get(r[ui], 1.0)
        seen = set()
        for (k, lid), m in sorted(per.items(), key=lambda kv: int(kv[0][1])):
            if k in seen:
                continue
            seen.add(k)
            t = m.get("gpu__time_duration.sum", 0)
            b = m.get("dram__bytes_read.sum", 0) + m.get("dram__bytes_write.sum", 0)
            gbs = b / t / 1e9 if t else 0
            loc = m.get("l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum", 0) + \
                m.get("l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum", 0)
            out.append("| %s | %s | %.3f | %.3f | %.1f | %.2f%% | %.1f%% | %.1f%% | %.1f%% | %.1f%% | %.3g |" % (
                wl, k.replace("void ", "")[:44], t * 1e3, b / 1e9, gbs, 100 * gbs / peak_gbs,
                100 * m.get("smsp__thread_inst_executed_per_inst_executed.ratio", 0) / 32,
                m.get("lts__t_sector_hit_rate.pct", 0), m.get("smsp__issue_active.avg.pct_of_peak_sustained_active", 0),
                m.get("sm__warps_active.avg.pct_of_peak_sustained_active", 0), loc))
    return "\n".join(out)


def eval_profiles(paths, outdir):
    """profiles/eval_inst_<wl>.json from a sweep capture: warp instructions and DRAM bytes of one launch of
    each eval-phase kernel (culi_eval*, culi_fanout_kernel), summed — the numbers bench.py's roofline uses."""
    for path in paths:
        wl = path.rsplit("_", 1)[-1].split(".")[0]
        rows = list(csv.reader(open(path, errors="replace")))
        hi = next(i for i, r in enumerate(rows) if "Metric Name" in r)
        h = rows[hi]
        ii, ki, mi, ui, vi = (h.index(x) for x in ("ID", "Kernel Name", "Metric Name", "Metric Unit", "Metric Value"))
        per = {}
        for r in rows[hi + 1:]:
            if len(r) > vi:
                per.setdefault((r[ki].split("(")[0], r[ii]), {})[r[mi]] = num(r[vi]) * UNIT.get(r[ui], 1.0)
        seen, inst, dram, t, kern = set(), 0.0, 0.0, 0.0, []
        for (k, lid), m in sorted(per.items(), key=lambda kv: int(kv[0][1])):
            if k in seen or not ("culi_eval" in k or "culi_fanout_kernel" in k):
                continue
            seen.add(k)
            kern.append(k.replace("void ", ""))
            inst += m.get("smsp__inst_executed.sum", 0)
            dram += m.get("dram__bytes_read.sum", 0) + m.get("dram__bytes_write.sum", 0)
            t += m.get("gpu__time_duration.sum", 0)
        out = {"source": path, "kernels": kern, "warp_inst_per_launch": inst, "dram_bytes": dram,
               "kernel_seconds_under_ncu": t}
        with open("%s/eval_inst_%s.json" % (outdir, wl.lower()), "w") as f:
            json.dump(out, f)
        print(wl, json.dumps(out))


def main():
    mode, path = sys.argv[1], sys.argv[2]
    if mode == "profiles":
        eval_profiles(sys.argv[3:], path)
        return
    if mode == "launches":
        print(launches(path))
        return
    if mode == "sweep":
        print(sweep(sys.argv[2:]))
        return
    res = full(path)
    for d in res:
        print("kernel:", d.pop("Kernel Name")[:100])
        for k, (v, u) in d.items():
            print("  %-70s %20s %s" % (k, v, u))
    if "--json" in sys.argv:
        d = full(path)[0]
        t = num(d["gpu__time_duration.sum"][0])
        tu = d["gpu__time_duration.sum"][1]
        scale = {"ns": 1e-9, "us": 1e-6, "usecond": 1e-6, "ms": 1e-3, "msecond": 1e-3, "s": 1}.get(tu, 1e-9)

        def byt(key):
            v, u = d[key]
            return num(v) * {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}.get(u, 1)
        out = {"source": path, "warp_inst_per_launch": num(d["smsp__inst_executed.sum"][0]),
               "dram_bytes": byt("dram__bytes_read.sum") + byt("dram__bytes_write.sum"),
               "kernel_seconds_under_ncu": t * scale,
               "thread_inst_per_warp_inst": num(d["smsp__thread_inst_executed_per_inst_executed.ratio"][0]),
               "l2_hit_pct": num(d["lts__t_sector_hit_rate.pct"][0]),
               "issue_active_pct": num(d["smsp__issue_active.avg.pct_of_peak_sustained_active"][0])}
        with open(sys.argv[sys.argv.index("--json") + 1], "w") as f:
            json.dump(out, f, indent=1)
        print(json.dumps(out))


if __name__ == "__main__":
    main()
