"""Multi-GPU driver for the CuLi hot path: shard, environment broadcast, gather.

One process per GPU (torchrun), `torch.distributed` for the collectives (NCCL over NVLink on the GPU box;
gloo in the CPU tests).  The collectives move opaque byte buffers produced and consumed by libculi.so:
  * culi_env_export / culi_env_import  — the global environment (persistent heap segment, global frame,
    strings, symbol names), broadcast from rank 0 once per session;
  * culi_results_serialize / culi_results_merge — per-rank results gathered to every rank and rebuilt in
    global form order (symbols re-interned by name).
  * culi_results_export / culi_results_import — the device-resident gather (the default): each rank packs
    its records + payload + names into a fixed-size device buffer (no host sync), one all_gather of the
    padded buffers (NCCL: device to device over NVLink), and the destination rank merges them on its GPU
    (records scattered by form index, payload offsets shifted, symbols re-interned) with one D2H.
No collective runs inside the eval kernel: the path has one exchange before and one after the batch.
"""
from __future__ import annotations

import torch
import torch.distributed as dist


def shard_indices(nforms: int, rank: int, world: int) -> list[int]:
    """Strided dealing: rank r takes forms {i : i mod world == r}."""
    return list(range(rank, nforms, world))


def _buffer_device(group=None) -> torch.device:
    backend = dist.get_backend(group)
    if backend == "nccl":
        return torch.device("cuda", torch.cuda.current_device())
    return torch.device("cpu")


def broadcast_bytes(payload: bytes | None, src: int = 0, group=None) -> bytes:
    """Broadcast a byte string from `src` (size first, then the bytes)."""
    dev = _buffer_device(group)
    rank = dist.get_rank(group)
    size = torch.zeros(1, dtype=torch.int64, device=dev)
    if rank == src:
        size[0] = len(payload)
    dist.broadcast(size, src, group=group)
    buf = torch.empty(int(size.item()), dtype=torch.uint8, device=dev)
    if rank == src:
        buf.copy_(torch.frombuffer(bytearray(payload), dtype=torch.uint8))
    dist.broadcast(buf, src, group=group)
    return bytes(buf.cpu().numpy().tobytes())


def broadcast_env(ctx, src: int = 0, group=None) -> int:
    """Define on `src`, broadcast the packed environment on the device, import on the others.
    Returns the number of bytes broadcast.  NCCL: the buffer never leaves the GPU."""
    dev = torch.device("cuda", torch.cuda.current_device())
    rank = dist.get_rank(group)
    size = torch.zeros(1, dtype=torch.int64, device=_buffer_device(group))
    if rank == src:
        size[0] = ctx.env_export_size()
    dist.broadcast(size, src, group=group)
    n = int(size.item())
    buf = torch.empty(n, dtype=torch.uint8, device=dev)
    if rank == src:
        ctx.env_export(buf.data_ptr(), n)
    if _buffer_device(group).type == "cuda":
        dist.broadcast(buf, src, group=group)
    else:                                           # gloo: stage through host memory
        hb = buf.cpu()
        dist.broadcast(hb, src, group=group)
        buf.copy_(hb)
    if rank != src:
        torch.cuda.synchronize()
        ctx.env_import(buf.data_ptr(), n)
    return n


def all_gather_bytes(blob: bytes, group=None) -> list[bytes]:
    """All-gather variable-size byte strings: sizes first, then zero-padded payloads."""
    dev = _buffer_device(group)
    world = dist.get_world_size(group)
    n = torch.tensor([len(blob)], dtype=torch.int64, device=dev)
    sizes = [torch.zeros(1, dtype=torch.int64, device=dev) for _ in range(world)]
    dist.all_gather(sizes, n, group=group)
    mx = max(int(s.item()) for s in sizes)
    pad = torch.zeros(max(mx, 1), dtype=torch.uint8, device=dev)
    if blob:
        pad[: len(blob)] = torch.frombuffer(bytearray(blob), dtype=torch.uint8).to(dev)
    outs = [torch.empty(max(mx, 1), dtype=torch.uint8, device=dev) for _ in range(world)]
    dist.all_gather(outs, pad, group=group)
    return [bytes(o[: int(s.item())].cpu().numpy().tobytes()) for o, s in zip(outs, sizes)]


def gather_results(results, nforms: int, group=None):
    """Gather every rank's serialized results and rebuild the full batch in global form order."""
    from paper_conf_cluster_subdbn18_b200 import culi
    world = dist.get_world_size(group)
    blobs = all_gather_bytes(results.serialize(), group=group)
    idx = [shard_indices(nforms, r, world) for r in range(world)]
    return culi.merge_results(blobs, idx)


def all_gather_device(buf: torch.Tensor, group=None) -> torch.Tensor:
    """all_gather_into_tensor of equal-size device buffers; gloo (CPU tests) stages through host memory."""
    world = dist.get_world_size(group)
    out = torch.empty(world * buf.numel(), dtype=buf.dtype, device=buf.device)
    if _buffer_device(group).type == "cuda":
        dist.all_gather_into_tensor(out, buf, group=group)
    else:
        h = torch.empty(world * buf.numel(), dtype=buf.dtype)
        dist.all_gather_into_tensor(h, buf.cpu(), group=group)
        out.copy_(h)
    return out


def export_capacity(ctx, group=None, slack: float = 1.25) -> int:
    """Common export-buffer size: the largest exact size over the ranks, with room for payload growth."""
    dev = _buffer_device(group)
    n = torch.tensor([ctx.results_export_size()], dtype=torch.int64, device=dev)
    dist.all_reduce(n, op=dist.ReduceOp.MAX, group=group)
    return (int(int(n.item()) * slack) + 4095) // 4096 * 4096


def gather_results_device(ctx, cap: int, dst: int | None = 0, group=None, buf: torch.Tensor | None = None):
    """Device-resident gather of the current batch's results (strided shards).  Every rank
    exports into `cap` bytes, one all_gather, rank `dst` (every rank if None) imports.  Returns the merged
    Results on the importing rank(s), else None."""
    dev = torch.device("cuda", torch.cuda.current_device())
    world = dist.get_world_size(group)
    if buf is None:
        buf = torch.empty(cap, dtype=torch.uint8, device=dev)
    ctx.results_export(buf.data_ptr(), cap)
    if _buffer_device(group).type != "cuda":
        torch.cuda.synchronize()                 # gloo reads the buffer on the host
    out = all_gather_device(buf, group=group)
    if dst is not None and dist.get_rank(group) != dst:
        return None
    torch.cuda.synchronize()
    ptrs = [out.data_ptr() + r * cap for r in range(world)]
    return ctx.results_import(ptrs, [cap] * world, None)
