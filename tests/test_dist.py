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
