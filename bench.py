#!/usr/bin/env python3
"""bench.py — forms/sec and eval-steps/sec of the CuLi hot path on B200 (BASELINE.json `metric`).

One "step" = one pass of the whole hot path over one batch of synthetic input already resident in HBM:
dispatch (classify + sort), the eval kernel, result export, and (N > 1) the NCCL all-gather of the
result records.  Default workload: configs[1] = C2, 65,536 (fib n) forms with n in 15..22 per GPU
(weak scaling: every rank evaluates its own 65,536-form shard of an N x 65,536 batch; the global
environment is defined on rank 0 and broadcast over NCCL once per session).

  python bench.py [--gpus N] [--steps K] [--warmup W] [--workload C2] [--impl culi|reference]

`--impl reference` times the oracle (the plain recursive CPU interpreter, oracle/) on the host cores on a
bounded sample of the same workload (this tier has no runnable reference implementation).
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

from paper_conf_cluster_subdbn18_b200 import workloads as W  # noqa: E402

L2_FLUSH_BYTES = 512 << 20          # > 126 MB L2: flushed between timed iterations
PEAKS_PATH = os.path.join(ROOT, "MEASURED_PEAKS.json")
WORKLOADS = {
    "C0": lambda n_rank, rank: W.c0(4096),
    "C1": lambda n_rank, rank: W.c1(1024 * n_rank),
    "C2": lambda n_rank, rank: W.c2(65536 * n_rank),
    "C3": lambda n_rank, rank: W.c3(1 << 20),
    "C4": lambda n_rank, rank: W.c4(262144 * n_rank),
    "C5": lambda n_rank, rank: W.c5(16777216),
}
SCALING = {"C0": "replicas", "C1": "weak", "C2": "weak", "C3": "replicas", "C4": "weak", "C5": "strong"}


def bench_config(workload: str, world: int) -> dict:
    """The `config` object shared by the culi arm and the reference (oracle) arm."""
    if workload == "C0":
        return {"workload": "C0 (paper-shaped context, PAPER L703 Fig.15): (||| 4096 fib (5 ... 5)), "
                            "units = element applications", "parallelism": "dp%d" % world,
                "l2": "flushed between timed steps (512 MB write)"}
    idx = {"C1": 0, "C2": 1, "C3": 2, "C4": 3, "C5": 4}[workload]
    what = {"C1": "1,024 integer arithmetic forms", "C2": "65,536 (fib n) forms, n in 15..22",
            "C3": "(||| 1048576 f xs), closure + let + float", "C4": "262,144 macro forms",
            "C5": "16.8M mixed forms"}[workload]
    return {"workload": "%s (BASELINE configs[%d]): %s" % (workload, idx, what),
            "parallelism": "dp%d" % world, "l2": "flushed between timed steps (512 MB write)"}


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--workload", default=os.environ.get("CULI_WORKLOAD", "C2"))
    ap.add_argument("--impl", default="culi", choices=["culi", "reference"])
    ap.add_argument("--e2e-steps", type=int, default=3)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--flags", type=int, default=0)
    return ap.parse_args()


# ------------------------------------------------------------------------------------------------ clocks
class ClockSampler:
    """nvidia-smi clocks + throttle reasons sampled during the timed region (B200_PROFILING.md)."""

    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,"
         "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
         "clocks_event_reasons.sw_power_cap")

    def __init__(self, device: int):
        self.device = device
        self.samples = []
        self._stop = threading.Event()
        self._t = None

    def _nvml_handle(self):
        """NVML handle of the CUDA device (by PCI bus id, so CUDA_VISIBLE_DEVICES remapping is respected)."""
        import pynvml
        import torch
        pynvml.nvmlInit()
        try:
            p = torch.cuda.get_device_properties(self.device)
            bus = "%08x:%02x:%02x.0" % (p.pci_domain_id, p.pci_bus_id, p.pci_device_id)
            return pynvml, pynvml.nvmlDeviceGetHandleByPciBusId(bus.encode())
        except Exception:  # noqa: BLE001
            return pynvml, pynvml.nvmlDeviceGetHandleByIndex(self.device)

    def _nvml_sample(self):
        nv, h, mx, get_r = self._nv
        bits = (0x8, 0x40, 0x20, 0x4)         # hw_slowdown, hw_thermal, sw_thermal, sw_power_cap
        sm = nv.nvmlDeviceGetClockInfo(h, nv.NVML_CLOCK_SM)
        r = get_r(h)
        self.samples.append([str(sm), str(mx)] + ["Active" if r & b else "Not Active" for b in bits])

    def _run(self):
        # NVML every 5 ms (a 10-step C2 run gets ~130 samples; __enter__ / __exit__ add one sample each, so a
        # timed region shorter than the period still has two); nvidia-smi every 0.2 s if NVML is missing
        if self._nv:
            while not self._stop.wait(0.005):
                try:
                    self._nvml_sample()
                except Exception:  # noqa: BLE001
                    pass
            return
        self.source = "nvidia-smi 0.2 s"
        while not self._stop.is_set():
            try:
                out = subprocess.run(["nvidia-smi", "-i", str(self.device), "--query-gpu=" + self.Q,
                                      "--format=csv,noheader,nounits"], capture_output=True, text=True,
                                     timeout=5).stdout.strip()
                if out:
                    self.samples.append([x.strip() for x in out.split(",")])
            except Exception:  # noqa: BLE001
                pass
            self._stop.wait(0.2)

    def __enter__(self):
        self._nv = None
        try:
            nv, h = self._nvml_handle()
            get_r = getattr(nv, "nvmlDeviceGetCurrentClocksEventReasons", None) or \
                nv.nvmlDeviceGetCurrentClocksThrottleReasons
            self._nv = (nv, h, nv.nvmlDeviceGetMaxClockInfo(h, nv.NVML_CLOCK_SM), get_r)
            self.source = "nvml 5 ms"
            self._nvml_sample()
        except Exception:  # noqa: BLE001
            self._nv = None
        self._t = threading.Thread(target=self._run, daemon=True)
        self._t.start()
        return self

    def __exit__(self, *a):
        self._stop.set()
        self._t.join(timeout=10)
        if self._nv:
            try:
                self._nvml_sample()
            except Exception:  # noqa: BLE001
                pass

    def summary(self):
        if not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"]}
        sm = [float(s[0]) for s in self.samples if s[0].replace(".", "").isdigit()]
        mx = [float(s[1]) for s in self.samples if s[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[k] for s in self.samples for k in range(4)
                          if len(s) > 2 + k and s[2 + k].lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": reasons, "samples": len(self.samples), "source": getattr(self, "source", None)}


def host_cpu_info():
    """lscpu model, sockets and SMT of the host the oracle runs on."""
    info = {}
    try:
        out = subprocess.run(["lscpu"], capture_output=True, text=True, timeout=10).stdout
        kv = {k.strip(): v.strip() for k, _, v in (l.partition(":") for l in out.splitlines()) if v}
        info = {"model": kv.get("Model name"), "sockets": int(kv.get("Socket(s)", "0") or 0),
                "threads_per_core": int(kv.get("Thread(s) per core", "0") or 0),
                "cpus_online": kv.get("On-line CPU(s) list")}
    except Exception:  # noqa: BLE001
        pass
    return info


def host_cores():
    try:
        return len(os.sched_getaffinity(0))
    except Exception:  # noqa: BLE001
        return os.cpu_count() or 1


# ---------------------------------------------------------------------------------------- oracle legs
def cpu_sample(wl: W.Workload, max_forms: int):
    """A bounded, strided sample of the workload's forms (the same text the GPU evaluates)."""
    lines = wl.form_lines()
    if wl.units != wl.nforms:            # ||| workloads: a shorter map of the same closure
        return wl, "full workload (single ||| form)"
    stride = max(1, len(lines) // max_forms)
    sample = lines[::stride][:max_forms]
    return (W.Workload(wl.name, wl.defs, "\n".join(sample) + "\n", len(sample), len(sample), wl.seed),
            "every %d-th form of %s (%d of %d forms)" % (stride, wl.name, len(sample), len(lines)))


def run_oracle(wl: W.Workload, max_forms: int, threads: int):
    import oracle
    sample, desc = cpu_sample(wl, max_forms)
    s = oracle.Session()
    if sample.defs:
        s.define(sample.defs)
    r = s.eval_batch(sample.forms, nthreads=threads, want_output=False)
    return sample, desc, r


ORACLE_SAMPLE = {"C0": 4096, "C1": 1024, "C2": 4096, "C3": 1 << 20, "C4": 262144, "C5": 262144}


def reference_arm(args):
    """--impl reference: the oracle on the host cores, rank 0 only (others exit 0)."""
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return
    wl = WORKLOADS[args.workload](1, 0)
    threads = host_cores()
    times, steps_tot, units = [], 0, 0
    for it in range(args.warmup + args.steps):
        sample, desc, r = run_oracle(wl, ORACLE_SAMPLE[args.workload], threads)
        if it >= args.warmup:
            times.append(r.seconds)
            steps_tot += r.total_steps
            units += sample.units
    t = sum(times)
    value = units / t
    line = {
        "metric": "forms/sec", "value": value, "unit": "forms/s", "impl": "reference",
        "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": 1e3 * t / len(times), "higher_is_better": True, "scaling": SCALING[args.workload],
        "vs_baseline": None, "dtype": "int64+f64", "data": "synthetic",
        "eval_steps_per_sec": steps_tot / t,
        "config": dict(bench_config(args.workload, args.gpus), sample=desc),
        "cpu_baseline": dict({"value": value, "unit": "forms/s", "cores": threads, "kind": "oracle",
                              "sample": desc}, **host_cpu_info()),
        "e2e": {"value": value, "unit": "forms/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)


# ------------------------------------------------------------------------------------------- culi leg
def load_peaks():
    try:
        with open(PEAKS_PATH) as f:
            return json.load(f), "measured"
    except Exception:  # noqa: BLE001
        return {"hbm_gbs": 6650.0, "sm_max_mhz": 1965.0}, "fallback"


def load_inst_profile(workload: str):
    """Warp instructions per eval-kernel launch from the committed ncu capture (profiles/)."""
    p = os.path.join(ROOT, "profiles", "eval_inst_%s.json" % workload.lower())
    try:
        with open(p) as f:
            return json.load(f)
    except Exception:  # noqa: BLE001
        return None


def culi_arm(args):
    import torch
    import torch.distributed as dist
    from paper_conf_cluster_subdbn18_b200 import culi
    from paper_conf_cluster_subdbn18_b200 import build as B

    world = int(os.environ.get("WORLD_SIZE", "1"))
    # CULI_FORCE_DIST=1: take the N > 1 path (process group, NCCL environment broadcast, device-resident
    # result gather) even with one rank — exercises the collectives on a single GPU
    dist_on = world > 1 or os.environ.get("CULI_FORCE_DIST") == "1"
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if world != args.gpus:
        args.gpus = world
    # CULI_SHARE_DEVICE=1 + CULI_DIST_BACKEND=gloo: every rank on cuda:0 (exercises the N>1 path on one GPU)
    if os.environ.get("CULI_SHARE_DEVICE") == "1":
        local = 0
    backend = os.environ.get("CULI_DIST_BACKEND", "nccl")
    torch.cuda.set_device(local)
    if dist_on:
        if backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", local))
        else:
            dist.init_process_group(backend)
    cdev = torch.device("cuda", local) if backend == "nccl" else torch.device("cpu")   # collective buffers
    B.build()
    culi.load()
    dev = torch.device("cuda", local)
    # a dedicated (capturable) stream for the whole run: culi_eval_uploaded replays a CUDA graph on it
    stream = torch.cuda.Stream(device=dev)
    torch.cuda.set_stream(stream)

    # ---- workload + shard (rank r takes forms i mod k == r)
    wl = WORKLOADS[args.workload](world if SCALING[args.workload] == "weak" else 1, rank)
    if SCALING[args.workload] in ("weak", "strong") and world > 1:
        shard_text, shard_idx = W.shard_lines(wl.forms, rank, world)
    else:
        shard_text, shard_idx = wl.forms, list(range(wl.nforms))
    units_rank = wl.units if wl.units != wl.nforms else len(shard_idx)

    heap = 1 << 26 if args.workload in ("C1", "C2") else 1 << 30
    ctx = culi.Context(device=local, stream=stream.cuda_stream, heap_nodes=heap, flags=args.flags)

    # ---- define on rank 0, broadcast the environment over NCCL (a3 + a10)
    t_env = None
    if not dist_on:
        if wl.defs:
            ctx.define(wl.defs)
    else:
        from paper_conf_cluster_subdbn18_b200 import dist as D
        if rank == 0 and wl.defs:
            ctx.define(wl.defs)
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        env_bytes = D.broadcast_env(ctx, src=0)
        torch.cuda.synchronize()
        t_env = {"ms": 1e3 * (time.perf_counter() - t0), "bytes": env_bytes}

    # ---- read (host, outside the timed region) + upload (a1, a2)
    t0 = time.perf_counter()
    img = ctx.read(shard_text)
    t_read = time.perf_counter() - t0
    h = ctx.upload(img)
    flush = torch.empty(L2_FLUSH_BYTES, dtype=torch.uint8, device=dev)
    # N > 1: the step ends with the device-resident result gather: every rank packs records
    # + list payload + names into a fixed-size device buffer (culi_results_export, no host sync) and one
    # NCCL all_gather moves the padded buffers; rank 0 can merge them on its GPU (culi_results_import, the
    # e2e path below).  The capacity is the largest exact size over the ranks (+25 %), from one eval.
    xcap, xbuf, gathered = 0, None, None
    if dist_on:
        from paper_conf_cluster_subdbn18_b200 import dist as D
        ctx.eval_uploaded(h)
        xcap = D.export_capacity(ctx)
        xbuf = torch.empty(xcap, dtype=torch.uint8, device=dev)
        gathered = torch.empty(world * xcap, dtype=torch.uint8, device=dev)

    def step():
        ctx.eval_uploaded(h)
        if dist_on:
            ctx.results_export(xbuf.data_ptr(), xcap)
            if cdev.type == "cuda":
                dist.all_gather_into_tensor(gathered, xbuf)
            else:
                torch.cuda.synchronize()
                g = torch.empty(world * xcap, dtype=torch.uint8)
                dist.all_gather_into_tensor(g, xbuf.cpu())
                gathered.copy_(g)

    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize()
    res = ctx.fetch_results(h)                  # parity-relevant numbers of this exact batch
    total_steps, n_err = res.totals()
    wire_bytes = res.wire_bytes()
    # the timed step is culi_eval_uploaded alone: it must not need the work a fetch can add afterwards
    # (sequential fallback of undecidable ||| forms, eval + export re-run into a grown payload buffer)
    fb0, regrow0 = ctx.last_reruns()
    if fb0:
        raise SystemExit("bench: %d forms needed the sequential fallback; the timed step would omit it" % fb0)
    del res

    # ---- timed region: K steps, CUDA events on the launching stream, L2 flushed between steps
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True))
          for _ in range(args.steps)]
    eval_ms, disp_ms, exp_ms = [], [], []
    if dist_on:
        dist.barrier()
    torch.cuda.synchronize()
    with ClockSampler(local) as clk:
        for k in range(args.steps):
            flush.fill_(k & 0xff)
            ev[k][0].record(stream)
            step()
            ev[k][1].record(stream)
            ms3, kernels, high = ctx.last_timing()
            disp_ms.append(ms3[0])
            eval_ms.append(ms3[1])
            exp_ms.append(ms3[2])
        torch.cuda.synchronize()
    if dist_on:
        dist.barrier()
    chk = ctx.fetch_results(h)                  # the timed steps' own results: same totals, no re-runs
    assert chk.totals() == (total_steps, n_err) and ctx.last_reruns() == (0, 0), ctx.last_reruns()
    waits_gave_up = ctx.last_waits()[0]
    splits = ctx.last_splits()
    del chk
    step_ms = [a.elapsed_time(b) for a, b in ev]
    t_rank = sum(step_ms) / 1e3
    t_max = t_rank
    if dist_on:
        tt = torch.tensor([t_rank], dtype=torch.float64, device=cdev)
        dist.all_reduce(tt, op=dist.ReduceOp.MAX)
        t_max = float(tt.item())
        agg = torch.tensor([units_rank, total_steps], dtype=torch.float64, device=cdev)
        dist.all_reduce(agg)
        units_all, steps_all = float(agg[0].item()), float(agg[1].item())
    else:
        units_all, steps_all = float(units_rank), float(total_steps)
    value = units_all * args.steps / t_max
    steps_per_sec = steps_all * args.steps / t_max

    # ---- e2e: the public C-ABI from host TEXT (culi_eval_text: H2D of the text from pinned memory, device
    # read §8(f)2, dispatch + eval + export, D2H of records + payload), the call a user makes
    ctx.release(h)
    text_b = shard_text.encode()
    text_host = torch.frombuffer(bytearray(text_b), dtype=torch.uint8).pin_memory()
    h2d = len(text_b)

    def e2e_loop(run):
        ms, nbytes = [], 0
        for k in range(args.e2e_steps):
            a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            if dist_on:
                dist.barrier()
            a.record(stream)
            r = run()
            if r is not None:
                nbytes = r.wire_bytes()
            b.record(stream)
            torch.cuda.synchronize()
            ms.append(a.elapsed_time(b))
            del r
        t = sum(ms) / 1e3
        if dist_on:
            tt = torch.tensor([t], dtype=torch.float64, device=cdev)
            dist.all_reduce(tt, op=dist.ReduceOp.MAX)
            t = float(tt.item())
        return units_all * len(ms) / t, 1e3 * t / len(ms), nbytes

    def e2e_text():
        if not dist_on:
            return ctx.eval_text(text_host)
        # N > 1: device read + eval of this rank's shard, device-resident gather, merge on rank 0's GPU,
        # one D2H of the whole batch's results there (no Python bytes on the path)
        hh, _nf = ctx.upload_text(text_host)
        ctx.eval_uploaded(hh)
        ctx.complete(hh)
        merged = D.gather_results_device(ctx, xcap, dst=0)
        ctx.release(hh)
        return merged

    ctx.eval_text(text_host)                         # warm the reader's buffers
    e2e_value, e2e_ms_step, d2h = e2e_loop(e2e_text)
    # the same through a host-read image (culi_read outside the timed region, culi_eval_batch inside)
    img_h2d = img.pin()
    img_value, img_ms_step = None, None
    if not dist_on:
        img_value, img_ms_step, _ = e2e_loop(lambda: ctx.eval_batch(img))

    # ---- device reader alone (§8(f)2): text resident in HBM -> node image in the heap
    text_dev = text_host.to(dev)
    rd_ms = []
    for _ in range(3):
        hh, _nf = ctx.upload_text(text_dev)
        rd_ms.append(ctx.last_read()[0])
        ctx.release(hh)
    _, rd_items, rd_nodes = ctx.last_read()
    rd_s = statistics.median(rd_ms) / 1e3
    peaks0, _src0 = load_peaks()
    rd_alg = len(text_b) + 9 * rd_nodes + 4 * len(shard_idx)     # text read once + image written once
    reader = {"ms": 1e3 * rd_s, "text_bytes": len(text_b), "items": rd_items, "nodes": rd_nodes,
              "host_read_ms": 1e3 * t_read, "text_gbs": len(text_b) / rd_s / 1e9,
              "roofline": {"bound": "hbm", "algorithmic_bytes": rd_alg, "achieved": rd_alg / rd_s / 1e9,
                           "peak": peaks0["hbm_gbs"], "unit": "GB/s",
                           "frac": rd_alg / rd_s / 1e9 / peaks0["hbm_gbs"]},
              "timing": "CUDA events around the whole read incl. its 3 host sync points (culi_last_read)"}

    if rank != 0:
        if dist_on:
            dist.barrier()
            dist.destroy_process_group()
        return

    # ---- roofline of the dominant kernel (the eval kernel; for ||| workloads plus the fan-out kernel)
    # the algorithmic HBM fraction = (bytes the method must move) / eval time / peak HBM.
    # Algorithmic bytes of one launch = the batch image read once (9 B per node, SURVEY §8 canonical
    # node) + the results written once (18 B record per form + 16 B per serialized list token, exactly
    # the fetched bytes) + for ||| workloads each element's cell and value read from the environment
    # (2 x 9 B).  C2: 4 nodes/form -> 36 + 18 = 54 B/form (§8(d): "52 B").  The kernel is in fact
    # bound by instruction issue / latency (an interpreter); the issue-slot view is its own field.
    peaks, peak_src = load_peaks()
    eval_s = statistics.mean(eval_ms) / 1e3
    clocks = clk.summary()
    prof = load_inst_profile(args.workload)
    image_bytes = 9 * img.nnodes
    env_bytes = 18 * wl.units if wl.units != wl.nforms else 0
    alg_bytes = image_bytes + wire_bytes + env_bytes
    hbm_ach = alg_bytes / eval_s / 1e9
    sm_mhz = peaks.get("sm_max_mhz", 1965.0)
    peak_inst = 148 * 4 * sm_mhz * 1e6 / 1e9          # G warp-instructions / s
    inst = prof.get("warp_inst_per_launch") if prof else None
    ach = inst / eval_s / 1e9 if inst else None
    roof = {"bound": "hbm", "achieved": hbm_ach, "peak": peaks["hbm_gbs"], "unit": "GB/s",
            "frac": hbm_ach / peaks["hbm_gbs"],
            "traffic": prof.get("dram_bytes") if prof else None,
            "algorithmic_bytes": alg_bytes,
            "algorithmic_source": "image %d B (9 B x %d nodes) + results %d B (fetched records + tokens) + "
                                  "||| elements %d B, per eval launch / live eval-phase CUDA-event time"
                                  % (image_bytes, img.nnodes, wire_bytes, env_bytes),
            "peak_source": "MEASURED_PEAKS.json hbm_gbs (%s)" % peak_src,
            "traffic_source": ("ncu dram__bytes_read.sum + dram__bytes_write.sum per launch "
                               "(profiles/eval_inst_%s.json)" % args.workload.lower()) if prof else None,
            "issue": {"achieved": ach, "peak": peak_inst, "unit": "Gwarp-inst/s",
                      "frac": (ach / peak_inst) if ach else None,
                      "peak_source": "148 SMs x 4 SMSP x 1 warp-inst/clk x %.0f MHz (B200_PROFILING.md)" % sm_mhz,
                      "source": ("ncu smsp__inst_executed.sum per launch (profiles/eval_inst_%s.json) / "
                                 "live eval-phase time" % args.workload.lower()) if inst else None}}

    cpu = None
    if world == 1 and not args.no_cpu_baseline:
        threads = host_cores()
        sample, desc, r = run_oracle(wl, ORACLE_SAMPLE[args.workload], threads)
        cpu = dict({"value": sample.units / r.seconds, "unit": "forms/s", "cores": threads, "kind": "oracle",
                    "sample": desc, "eval_steps_per_sec": r.total_steps / r.seconds}, **host_cpu_info())

    ms_step = 1e3 * t_max / args.steps
    line = {
        "metric": "forms/sec", "value": value, "unit": "forms/s", "n_gpus": world, "steps": args.steps,
        "warmup": args.warmup, "ms_per_step": ms_step, "higher_is_better": True,
        "scaling": SCALING[args.workload] if world > 1 else "weak", "vs_baseline": None,
        "dtype": "int64+f64", "data": "synthetic",
        "eval_steps_per_sec": steps_per_sec,
        "config": dict(bench_config(args.workload, world), forms_per_gpu=len(shard_idx),
                       units_per_gpu=units_rank, binning=not (args.flags & 1)),
        "gpu_launches": kernels * args.steps,
        "phases_ms": {"dispatch": statistics.mean(disp_ms), "eval": statistics.mean(eval_ms),
                      "export": statistics.mean(exp_ms)},
        "errors_in_batch": n_err, "read_s": t_read, "env_broadcast_ms": t_env,
        "split_groups": splits, "waits_gave_up": waits_gave_up, "fallback_forms": 0, "payload_regrows": 0,
        "roofline": roof,
        "cpu_baseline": cpu,
        "e2e": {"value": e2e_value, "unit": "forms/s", "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": d2h,
                "ms_per_step": e2e_ms_step,
                "path": ("culi_eval_text: pinned host text -> read (device reader; the host reader for texts of "
                         "<= 16 KiB) -> eval -> host results" if not dist_on
                         else "per rank: pinned host text -> device read -> eval -> culi_results_export -> NCCL "
                              "all_gather; rank 0: culi_results_import (device merge) -> host results")},
        "e2e_image": {"value": img_value, "unit": "forms/s", "h2d_bytes_per_step": img_h2d,
                      "ms_per_step": img_ms_step, "path": "culi_eval_batch on a host-read image"},
        "reader": reader,
        "clocks": clocks,
    }
    print(json.dumps(line), flush=True)
    if dist_on:
        dist.barrier()
        dist.destroy_process_group()


def main():
    args = parse()
    if args.impl == "reference":
        reference_arm(args)
    else:
        culi_arm(args)


if __name__ == "__main__":
    main()
