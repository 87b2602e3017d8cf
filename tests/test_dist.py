"""CPU tests of the multi-GPU host logic (LPT sharding + the final reduction)
with the gloo backend, world_size 2. The per-shard results come
from the oracle (standing in for each GPU's grep); the reduced result must equal
the oracle run on the whole corpus."""
import os
import socket

import numpy as np
import pytest
import torch.multiprocessing as mp

import gen
import oracle
from paper_conf_asplos_silbersteinfkw13_b200 import dist as gdist


def test_lpt_balanced_and_complete():
    rng = np.random.default_rng(0)
    sizes = rng.lognormal(np.log(7000), 1.3, size=3000).astype(np.int64)
    for n in (1, 2, 4, 8):
        sh = gdist.lpt_shard(sizes, n)
        allidx = sorted(i for s in sh for i in s)
        assert allidx == list(range(len(sizes)))
        loads = [int(sizes[s].sum()) for s in sh]
        assert max(loads) - min(loads) <= int(sizes.max())  # LPT bound


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, ws, port, corpus, outdir):
    import torch.distributed as dist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=ws)
    sizes = [os.path.getsize(p) for p in corpus["paths"]]
    shard = gdist.lpt_shard(sizes, ws)[rank]
    lst = gdist.write_shard_list(corpus["paths"], shard, os.path.join(outdir, f"shard{rank}.txt"))
    r = oracle.grep(corpus["dict"], lst, want_hits=False)
    recs = gdist.globalize_records(r.records, shard)
    # digest terms depend on the file index: recompute with global indices via the oracle on
    # one-file lists is not needed for the reduction test; compare totals/records/hit count
    tot, dig, allrecs = gdist.reduce_grep(dist.group.WORLD, r.totals, r.digest, recs)
    if rank == 0:
        np.save(os.path.join(outdir, "tot.npy"), tot)
        np.save(os.path.join(outdir, "recs.npy"), allrecs)
        np.save(os.path.join(outdir, "nh.npy"), np.array([dig[2]]))
    dist.barrier()
    dist.destroy_process_group()


def test_gloo_world2_reduce_equals_whole(shmdir):
    c = gen.c4_corpus(os.path.join(shmdir, "c4"), seed=9, nfiles=200, total_bytes=2 << 20, nwords=3000)
    mp.spawn(_worker, args=(2, _free_port(), c, shmdir), nprocs=2, join=True)
    whole = oracle.grep(c["dict"], c["list"], want_hits=False)
    assert np.load(os.path.join(shmdir, "tot.npy")).tolist() == whole.totals.tolist()
    assert np.load(os.path.join(shmdir, "recs.npy")).tolist() == whole.records.tolist()
    assert int(np.load(os.path.join(shmdir, "nh.npy"))[0]) == whole.digest[2]


def _worker_rows(rank, ws, port, m, outdir):
    import torch
    import torch.distributed as dist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=ws)
    rows, cols = m["rows"], m["cols"]
    r0, r1 = gdist.row_block(rows, ws, rank)
    ys = torch.as_tensor(oracle.matvec(m["A"], m["x"], rows, cols, row0=r0, nrows=r1 - r0).astype(np.float32))
    y = gdist.gather_rows(dist.group.WORLD, ys, rows)
    # records gathered to rank 0 only
    recs = np.array([[rank, 1, 2]], dtype=np.uint64)
    _, _, got = gdist.reduce_grep(dist.group.WORLD, np.zeros(3, np.uint64), (rank, 0, 1), recs, root=0)
    np.save(os.path.join(outdir, f"y{rank}.npy"), y.numpy())
    np.save(os.path.join(outdir, f"r{rank}.npy"), got)
    dist.barrier()
    dist.destroy_process_group()


@pytest.mark.parametrize("ws", [2, 3])
def test_gloo_row_split_gather_equals_whole(shmdir, ws):
    """C3 row blocks (one per rank) + all-gather == the whole product; grep records
    gathered to rank 0 only (the bench's multi-GPU plumbing)."""
    m = gen.matrix_files(os.path.join(shmdir, "mv"), 37, 96, seed=5)
    mp.spawn(_worker_rows, args=(ws, _free_port(), m, shmdir), nprocs=ws, join=True)
    whole = oracle.matvec(m["A"], m["x"], 37, 96).astype(np.float32)
    for r in range(ws):
        assert np.array_equal(np.load(os.path.join(shmdir, f"y{r}.npy")), whole)
    assert np.load(os.path.join(shmdir, "r0.npy")).tolist() == [[r, 1, 2] for r in range(ws)]
    for r in range(1, ws):
        assert len(np.load(os.path.join(shmdir, f"r{r}.npy"))) == 0


def test_split_helpers_cover_everything():
    for n in (1, 2, 3, 8):
        blocks = [gdist.row_block(11200, n, r) for r in range(n)]
        assert blocks[0][0] == 0 and blocks[-1][1] == 11200
        assert all(blocks[i][1] == blocks[i + 1][0] for i in range(n - 1))
        size, P = (8 << 30) + 12345, 2 << 20
        rngs = [gdist.byte_range(size, n, r, P) for r in range(n)]
        assert rngs[0][0] == 0 and sum(x[1] for x in rngs) == size
        assert all(rngs[i][0] + rngs[i][1] == rngs[i + 1][0] for i in range(n - 1))
        assert all(x[0] % P == 0 for x in rngs)
