"""bench.py's multi-rank path end to end on a one-GPU box: two ranks launched
by torch.distributed.run share cuda:0 with the test-only host-staged halo
transport (NCCL refuses two ranks on one GPU).  Everything else is the path
the driver's N-GPU run takes: the slab partition (weak and strong scaling),
the deep-halo schedule, the max-over-ranks timing, the halo metrics and the
one JSON line printed by rank 0."""
import json
import os
import socket
import subprocess
import sys

import pytest

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _run(*args):
    env = dict(os.environ)
    for k in ("WORLD_SIZE", "RANK", "LOCAL_RANK", "MASTER_ADDR", "MASTER_PORT"):
        env.pop(k, None)
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2", "--master-addr",
           "127.0.0.1", "--master-port", str(_port()), os.path.join(ROOT, "bench.py"), "--gpus", "2",
           "--test-transport", "staged", "--steps", "1", "--warmup", "3", "--no-cpu"] + list(args)
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=900, env=env, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [json.loads(ln) for ln in r.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, r.stdout[-2000:]            # rank 0 alone prints
    return lines[0]


def test_bench_two_ranks_weak_j3d7():
    d = _run()
    assert d["n_gpus"] == 2 and d["scaling"] == "weak"
    assert d["config"]["global_extents"] == [1024, 512, 512] and d["config"]["extents_per_gpu"] == [512, 512, 512]
    assert d["config"]["halo_depth"] == 4 and d["config"]["parallelism"] == "slab-z x2"
    h = d["halo"]
    assert h["ghost_planes"] == 4 and h["neighbours"] == 1
    assert h["bytes_per_neighbour_per_exchange"] == 4 * 512 * 512 * 4
    assert h["exchanges_per_100_time_steps"] == 25 and h["exchange_us"] > 0
    assert d["value"] > 0 and d["e2e"]["value"] > 0
    # 25 blocks of 4 steps, each two-step pass (K2R) + the last pair as
    # boundary low, boundary high and interior passes
    assert d["gpu_launches"] == 1 * 25 * 4
    assert d["roofline"]["time_steps_per_launch"] == 2


def test_bench_two_ranks_strong_acoustic13_depth1():
    d = _run("--workload", "acoustic13_1024", "--scaling", "strong", "--halo-depth", "1", "--no-e2e")
    assert d["scaling"] == "strong" and d["config"]["extents_per_gpu"] == [512, 1024, 1024]
    h = d["halo"]
    assert h["ghost_planes"] == 2 and h["grids_per_exchange"] == 1
    assert h["exchanges_per_100_time_steps"] == 100
