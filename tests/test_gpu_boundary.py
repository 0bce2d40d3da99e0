"""GPU tests of the SURVEY §8(b) boundary calls added in round 2: culi_eval_batch_async / culi_sync (the
paper's host-reads / device-evaluates split), a caller-owned device arena
(culi_opts.heap_base from a torch tensor), and the device-resident result export / import used by the
multi-GPU gather (PAPER L584-589 ordered result assembly) — all against the oracle."""
from __future__ import annotations

import pytest

from paper_conf_cluster_subdbn18_b200 import workloads as W
from tests.parity import compare
from tests.test_gpu_parity import SMALL, culi  # noqa: F401  (fixture)

pytestmark = pytest.mark.gpu

DEFS = "\n".join([W.FIB_DEF, W.FACT_DEF, W.SUM_DEF, W.WHEN_DEF, "(define greeting \"hello world\")"])
EXTRA = ["greeting", "'local-sym", "(list 'a \"s\" 1.5 (list 'b))", "(car 5)", "(||| 3 fib '(5 6 7))",
         "(cons 'x 'y)", "nil"]


def _oracle(oracle_mod, defs, forms):
    s = oracle_mod.Session()
    s.define(defs)
    return s.eval(forms)


def test_async_then_sync(culi, oracle_mod):
    wl = W.c5(3000, seed=21)
    forms = wl.forms + "\n".join(EXTRA) + "\n"
    defs = wl.defs + "\n" + DEFS
    ctx = culi.Context(**SMALL)
    ctx.define(defs)
    r = ctx.eval_batch_async(forms)
    nxt = ctx.read(W.c1(500).forms)              # the host reads the next batch while the device evaluates
    with pytest.raises(culi.CuliError) as ei:     # not ready before culi_sync
        r.info(0)
    assert ei.value.status == -7
    assert len(r) == 0
    with pytest.raises(culi.CuliError):           # one batch in flight per ctx
        ctx.eval_batch_async(forms)
    ctx.sync()
    o = _oracle(oracle_mod, defs, forms)
    assert not compare(r.printed(), r.steps(), o, forms.splitlines())
    r2 = ctx.eval_batch(nxt)                      # the ctx is usable again
    assert len(r2) == 500
    ctx.sync()                                    # no batch in flight: a no-op


def test_async_results_freed_before_sync(culi):
    ctx = culi.Context(**SMALL)
    ctx.define(W.FIB_DEF)
    r = ctx.eval_batch_async("(fib 20)\n" * 100)
    del r                                         # culi_results_free completes the batch first
    assert ctx.eval_batch("(fib 10)").printed() == ["55"]


def test_caller_owned_arena(culi, oracle_mod):
    import torch
    kw = dict(heap_nodes=1 << 22, vstack_entries=1024, slots=148 * 128)
    need = culi.Context.arena_bytes(**kw)
    arena = torch.empty(need, dtype=torch.uint8, device="cuda")
    ctx = culi.Context(arena=arena, **kw)
    wl = W.c5(2000, seed=5)
    ctx.define(wl.defs)
    r = ctx.eval_batch(wl.forms)
    assert not compare(r.printed(), r.steps(), _oracle(oracle_mod, wl.defs, wl.forms))
    # the heap really lives in the caller's tensor: the nil / T nodes at its start (16-byte nodes
    # {word u64, tag u8, pad}) carry tags 0 and 1
    assert arena[8].item() == 0 and arena[24].item() == 1 and arena[:8].tolist() == [0] * 8
    small = torch.empty(need - 4096, dtype=torch.uint8, device="cuda")
    with pytest.raises(culi.CuliError) as ei:
        culi.Context(arena=small, **kw)
    assert ei.value.status == -1


def test_export_import_single_and_virtual_ranks(culi, oracle_mod):
    """Shards of one batch evaluated in separate contexts (virtual ranks on one GPU), exported to device
    buffers and merged by culi_results_import — strided (form_index NULL) and with explicit indices."""
    import torch
    wl = W.c5(2500, seed=9)
    forms = wl.forms + "\n".join(EXTRA) + "\n"
    defs = wl.defs + "\n" + DEFS
    o = _oracle(oracle_mod, defs, forms)
    lines = forms.splitlines()
    world = 3
    ctxs, bufs, caps, idxs = [], [], [], []
    for r in range(world):
        ctx = culi.Context(**SMALL)
        ctx.define(defs)
        shard, idx = W.shard_lines(forms, r, world)
        h = ctx.upload(shard)
        ctx.eval_uploaded(h)
        ctx.complete(h)
        cap = ctx.results_export_size()
        buf = torch.empty(cap + 4096, dtype=torch.uint8, device="cuda")
        used = ctx.results_export(buf.data_ptr(), buf.numel())
        assert used >= cap
        ctxs.append(ctx)
        bufs.append(buf)
        caps.append(buf.numel())
        idxs.append(idx)
    torch.cuda.synchronize()
    ptrs = [b.data_ptr() for b in bufs]
    m1 = ctxs[0].results_import(ptrs, caps, None)
    assert not compare(m1.printed(), m1.steps(), o, lines)
    # explicit indices, ranks given in another order
    perm = [2, 0, 1]
    m2 = ctxs[1].results_import([ptrs[k] for k in perm], [caps[k] for k in perm], [idxs[k] for k in perm])
    assert (m2.printed(), m2.steps()) == (m1.printed(), m1.steps())
    # one rank alone == its own fetch
    f0 = ctxs[0].fetch_results(1)
    m0 = ctxs[0].results_import([ptrs[0]], [caps[0]], [list(range(len(idxs[0])))])
    assert (m0.printed(), m0.steps()) == (f0.printed(), f0.steps())
    # an export too small for the payload is flagged and refused by the import
    small_cap = ctxs[0].results_export_size() - 64
    sb = torch.empty(small_cap, dtype=torch.uint8, device="cuda")
    ctxs[0].results_export(sb.data_ptr(), small_cap)
    torch.cuda.synchronize()
    with pytest.raises(culi.CuliError):
        ctxs[0].results_import([sb.data_ptr()], [small_cap], [idxs[0]])
    for c in ctxs:
        c.release(1)
