"""a10 on a real GPU: two ranks (gloo process group, both on cuda:0 — the gpurun box has one GPU) run the
distributed path bench.py uses: rank 0 defines, the packed environment is broadcast and imported, each
rank evaluates its strided shard, results are gathered and merged in global form order, and the merged
batch must match the oracle element by element."""
from __future__ import annotations

import os
import socket

import pytest
import torch.multiprocessing as mp

pytestmark = pytest.mark.gpu


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, defs, forms, q):
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    sys.path.insert(0, root)
    import torch
    import torch.distributed as dist
    from paper_conf_cluster_subdbn18_b200 import culi, workloads as W, dist as D
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        torch.cuda.set_device(0)
        culi.load()
        ctx = culi.Context(device=0, stream=torch.cuda.current_stream().cuda_stream, slots=148 * 128,
                           heap_nodes=1 << 24, vstack_entries=2048)
        if rank == 0:
            ctx.define(defs)
        nbytes = D.broadcast_env(ctx, src=0)
        nforms = len(forms.splitlines())
        shard, idx = W.shard_lines(forms, rank, world)
        assert idx == D.shard_indices(nforms, rank, world)
        res = ctx.eval_batch(shard)
        merged = D.gather_results(res, nforms)               # host-serialized blobs (reference path)
        # device-resident gather (culi_results_export / culi_results_import): no Python bytes
        h = ctx.upload(shard)
        ctx.eval_uploaded(h)
        ctx.complete(h)
        cap = D.export_capacity(ctx)
        dm = D.gather_results_device(ctx, cap, dst=None)
        ctx.release(h)
        q.put((rank, nbytes, merged.printed(), merged.steps(), dm.printed(), dm.steps()))
    finally:
        dist.destroy_process_group()


@pytest.mark.timeout(300)
def test_two_ranks_broadcast_shard_gather(oracle_mod):
    import torch
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_cluster_subdbn18_b200 import build, workloads as W
    from tests.parity import compare
    build.build()
    wl = W.c5(3000)
    defs = wl.defs + "\n(define xs '(1 2 3))\n(define greeting \"hello\")\n"
    forms = wl.forms + "xs\ngreeting\n(||| 3 fib xs)\nlocal-symbol\n"
    world = 2
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_worker, args=(r, world, port, defs, forms, q)) for r in range(world)]
    for p in procs:
        p.start()
    outs = [q.get(timeout=280) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    s = oracle_mod.Session()
    s.define(defs)
    o = s.eval(forms)
    for rank, nbytes, printed, steps, dprinted, dsteps in outs:
        assert nbytes > 0
        bad = compare(printed, steps, o, forms.splitlines())
        assert not bad, "\n".join(bad)
        assert (dprinted, dsteps) == (printed, steps)


@pytest.mark.timeout(600)
def test_bench_nccl_path_single_rank():
    """bench.py's N > 1 path with the NCCL backend for real (one rank: the box has one GPU; CULI_FORCE_DIST):
    process group over NCCL, environment broadcast, device-resident export + all_gather_into_tensor in the
    timed step, the e2e gather + device merge on rank 0; the line must carry the distributed e2e path."""
    import json
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, CULI_FORCE_DIST="1")
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "1",
           "--master-addr", "127.0.0.1", "--master-port", str(_free_port()), os.path.join(root, "bench.py"),
           "--gpus", "1", "--workload", "C2", "--steps", "2", "--warmup", "3", "--e2e-steps", "1",
           "--no-cpu-baseline"]
    out = subprocess.run(cmd, capture_output=True, text=True, env=env, cwd=root, timeout=540)
    assert out.returncode == 0, out.stderr[-3000:]
    line = json.loads([x for x in out.stdout.splitlines() if x.startswith("{")][-1])
    assert line["value"] > 0 and line["waits_gave_up"] == 0
    assert "all_gather" in line["e2e"]["path"] and line["env_broadcast_ms"]["bytes"] > 0
