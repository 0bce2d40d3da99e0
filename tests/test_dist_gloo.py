"""The N>1 path on CPU: world_size-2 gloo process group exercising the same driver code bench.py uses
(paper_conf_cluster_subdbn18_b200/dist.py): strided sharding, byte broadcast (environment), variable-size
all-gather of serialized results and the merge back into global form order."""
from __future__ import annotations

import os
import socket

import pytest
import torch.multiprocessing as mp

from tests import wire


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    sys.path.insert(0, root)
    import torch.distributed as dist
    from paper_conf_cluster_subdbn18_b200 import dist as D
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        nforms = 7
        mine = D.shard_indices(nforms, rank, world)
        env = D.broadcast_bytes(b"ENV" + bytes(range(200)) if rank == 0 else None, src=0)
        # each rank "evaluates" its shard: form i -> INT i*i, with a rank-local symbol for form 5
        extra = ["r%d" % rank]
        recs = []
        for i in mine:
            if i == 5:
                recs.append((wire.SYM, 0, 1, wire.sym_id("r%d" % rank, extra)))
            else:
                recs.append((wire.INT, 0, i + 1, i * i))
        blob = wire.blob(recs, names=extra)
        blobs = D.all_gather_bytes(blob)
        from paper_conf_cluster_subdbn18_b200 import culi
        culi.load()
        m = culi.merge_results(blobs, [D.shard_indices(nforms, r, world) for r in range(world)])
        q.put((rank, env[:3], len(env), m.printed(), m.steps()))
    finally:
        dist.destroy_process_group()


@pytest.mark.timeout(120)
def test_gloo_world2_shard_broadcast_gather():
    from paper_conf_cluster_subdbn18_b200 import build
    build.build()
    world = 2
    port = _free_port()
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    outs = [q.get(timeout=100) for _ in range(world)]
    for p in procs:
        p.join(timeout=30)
        assert p.exitcode == 0
    for rank, head, n, printed, steps in outs:
        assert head == b"ENV" and n == 203
        # form 5 lives on rank 1 (5 mod 2), whose local symbol is r1
        assert printed == ["0", "1", "4", "9", "16", "r1", "36"]
        assert steps == [1, 2, 3, 4, 5, 1, 7]


def test_shard_indices_partition():
    from paper_conf_cluster_subdbn18_b200 import dist as D
    for n in (0, 1, 5, 64, 1000):
        for world in (1, 2, 3, 8):
            parts = [D.shard_indices(n, r, world) for r in range(world)]
            flat = sorted(i for p in parts for i in p)
            assert flat == list(range(n))
            assert max(len(p) for p in parts) - min(len(p) for p in parts) <= 1
