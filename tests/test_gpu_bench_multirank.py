"""The bench's multi-rank path (one process per GPU) on a one-GPU box:
two ranks share cuda:0 over gloo (GFS_BENCH_ONE_GPU=1 test mode). Checks that every
phase runs, C5 maps the other rank's cache (peer fill replaces the host re-read)
and every parity flag the bench reports holds."""
import json
import os
import socket
import subprocess
import sys

import pytest

pytestmark = [pytest.mark.gpu, pytest.mark.timeout(900)]
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def test_bench_two_ranks_one_gpu():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    env = dict(os.environ, GFS_BENCH_ONE_GPU="1")
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2",
           "--master-addr", "127.0.0.1", "--master-port", str(port), "bench.py", "--gpus", "2", "--steps", "2",
           "--warmup", "3", "--file-gib", "1", "--cache-gib", "1", "--hit-file-gib", "1", "--hit-calls", "64",
           "--hg-gib", "1", "--reps", "2", "--grep-files", "2000", "--grep-mib", "20", "--mv-rows", "560",
           "--mv-passes", "1", "--c5-mib", "32", "--c5-iters", "2", "--no-fig4", "--ref-sample-mib", "64"]
    out = subprocess.run(cmd, cwd=ROOT, env=env, capture_output=True, text=True, timeout=800)
    assert out.returncode == 0, out.stderr[-3000:]
    lines = [l for l in out.stdout.splitlines() if l.startswith("{")]
    assert len(lines) == 1, out.stdout[-2000:]
    d = json.loads(lines[0])
    assert d["n_gpus"] == 2
    assert d["parity"]["c2_oracle_checksum_every_step_all_ranks"]
    assert d["c2_byte_split"]["parity"] and d["c2_byte_split"]["err"] == 0
    assert all(d["grep"]["parity"].values()), d["grep"]  # incl. the digest: global file ids at N = 2
    assert d["matvec"]["parity"]["ok"], d["matvec"]
    assert d["hit"]["parity"]["checksum_eq_oracle"]
    assert all(p["parity"] for p in d["hit_global"]["points"])
    assert all(d["c1"]["parity"].values())
    c5 = d["c5"]
    assert c5["parity"] == {"host_file": True, "reread_checksums": True}
    assert c5["peers_attached"] == 1 and c5["peer_error"] is None
    assert c5["counters"]["peer_fill"] > 0 and c5["counters"]["rpc_read"] == 0
    assert list(d)[-1] == "summary"
