"""Multi-GPU plumbing: one process per GPU, each with a private
GPUfs cache and a shard of the file set; the only collective is the final
reduction of results (NCCL over NVLink on B200, gloo in CPU tests).

The paper splits its input statically and equally across <= 4 GPUs
(P:L1222-1223); here files are assigned by LPT on their sizes (longest
processing time first: largest file to the least-loaded rank), which keeps the
byte load balanced for the lognormal file sizes of a source tree.
Sizes come from stat() metadata only; file contents are read on the GPUs.
"""
from __future__ import annotations

import heapq
import os

import numpy as np


def lpt_shard(sizes, nranks: int) -> list[list[int]]:
    """Indices of files per rank, LPT by size; each rank's indices ascending."""
    if nranks < 1:
        raise ValueError("nranks must be >= 1")
    order = sorted(range(len(sizes)), key=lambda i: (-int(sizes[i]), i))
    heap = [(0, r) for r in range(nranks)]
    out: list[list[int]] = [[] for _ in range(nranks)]
    for i in order:
        load, r = heapq.heappop(heap)
        out[r].append(i)
        heapq.heappush(heap, (load + int(sizes[i]), r))
    return [sorted(x) for x in out]


def row_block(rows: int, nranks: int, rank: int) -> tuple[int, int]:
    """The contiguous row block [r0, r1) of `rank` in the C3 row split."""
    return rows * rank // nranks, rows * (rank + 1) // nranks


def byte_range(size: int, nranks: int, rank: int, align: int) -> tuple[int, int]:
    """The byte range [off, off + n) of `rank` in the C2 split of one file (§8(e)):
    equal `align`-multiple pieces, the last rank takes the rest."""
    per = (size // nranks) // align * align
    off = rank * per
    return off, (size - off if rank == nranks - 1 else per)


def gather_rows(pg_world, y_shard, rows: int, device=None):
    """All-gather of the ranks' y shards (NCCL / gloo all_gather of zero-padded
    equal-size buffers): the whole y, in row order, on every rank."""
    import torch
    import torch.distributed as dist
    ws = dist.get_world_size(pg_world) if (pg_world is not None and dist.is_initialized()) else 1
    if ws == 1:
        return y_shard
    per = (rows + ws - 1) // ws
    dev = device if device is not None else y_shard.device
    yp = torch.zeros(per, dtype=y_shard.dtype, device=dev)
    yp[:y_shard.numel()] = y_shard
    parts = [torch.zeros_like(yp) for _ in range(ws)]
    dist.all_gather(parts, yp, group=pg_world)
    return torch.cat([parts[r][:row_block(rows, ws, r)[1] - row_block(rows, ws, r)[0]] for r in range(ws)])


def write_shard_list(paths, idx, out_path: str) -> str:
    """List file for one shard (absolute paths, one per line)."""
    tmp = out_path + f".tmp{os.getpid()}"
    with open(tmp, "w") as f:
        for i in idx:
            f.write(os.path.abspath(paths[i]) + "\n")
    os.replace(tmp, out_path)
    return out_path


def globalize_records(records: np.ndarray, shard_idx) -> np.ndarray:
    """Map shard-local file indices of (file, word, count) records to global ones."""
    if len(records) == 0:
        return records.reshape(0, 3).astype(np.uint64)
    m = np.asarray(shard_idx, dtype=np.uint64)
    r = records.astype(np.uint64).copy()
    r[:, 0] = m[r[:, 0].astype(np.int64)]
    return r


def reduce_grep(pg_world, totals, digest, records, device=None, root=None):
    """The final reduction: all-reduce (sum) of per-word totals, of the hit
    count and of the order-independent digest sum; all-gather of the XOR terms
    (8 bytes per rank); the (already global) record arrays gathered to `root`
    (or to every rank when root is None). Works for the NCCL and gloo backends;
    without a process group (one rank) returns the local values.
    Returns (totals, digest, records) — records empty on ranks other than root."""
    import torch
    import torch.distributed as dist
    if pg_world is None or not dist.is_initialized() or dist.get_world_size(pg_world) == 1:
        recs = np.asarray(records, dtype=np.uint64).reshape(-1, 3)
        if len(recs):
            recs = recs[np.lexsort((recs[:, 1], recs[:, 0]))]
        return (np.asarray(totals, dtype=np.uint64), (int(digest[0]), int(digest[1]), int(digest[2])), recs)
    dev = device if device is not None else torch.device("cpu")
    t = torch.as_tensor(np.asarray(totals, dtype=np.uint64).view(np.int64), device=dev).clone()
    dist.all_reduce(t, op=dist.ReduceOp.SUM, group=pg_world)
    s = torch.tensor([np.uint64(digest[0]).astype(np.int64), int(digest[2])], dtype=torch.int64, device=dev)
    dist.all_reduce(s, op=dist.ReduceOp.SUM, group=pg_world)
    ws = dist.get_world_size(pg_world)
    x = torch.tensor([np.uint64(digest[1]).astype(np.int64)], dtype=torch.int64, device=dev)
    xs = [torch.zeros_like(x) for _ in range(ws)]
    dist.all_gather(xs, x, group=pg_world)
    xor = np.uint64(0)
    for v in xs:
        xor ^= np.int64(v.item()).astype(np.uint64)
    mine = np.asarray(records, dtype=np.uint64)
    if root is None:
        objs = [None] * ws
        dist.all_gather_object(objs, mine, group=pg_world)
    else:
        objs = [None] * ws if dist.get_rank() == root else None
        dist.gather_object(mine, objs, dst=root, group=pg_world)
    if objs is not None:
        recs = np.concatenate([o for o in objs if len(o)]) if any(len(o) for o in objs) else np.zeros((0, 3), np.uint64)
        if len(recs):
            recs = recs[np.lexsort((recs[:, 1], recs[:, 0]))]
    else:
        recs = np.zeros((0, 3), np.uint64)
    tot = t.cpu().numpy().view(np.uint64)
    sv = s.cpu().numpy()
    return tot, (int(np.int64(sv[0]).astype(np.uint64)), int(xor), int(sv[1])), recs
