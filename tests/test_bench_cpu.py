"""bench.py's launcher on CPU (no GPU): ``--gpus N`` without a torchrun
environment re-executes through torch.distributed.run with N ranks, each rank
checks the world size; ``--gpus 2`` on a box without 2 GPUs errors instead of
timing one GPU; the all-core oracle baseline reports its cores and model."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
BENCH = os.path.join(ROOT, "bench.py")


def _env():
    env = dict(os.environ)
    for k in ("WORLD_SIZE", "RANK", "LOCAL_RANK", "MASTER_ADDR", "MASTER_PORT"):
        env.pop(k, None)
    return env


def test_bench_launcher_gloo():
    r = subprocess.run([sys.executable, BENCH, "--gpus", "2", "--selftest-launch"], capture_output=True, text=True,
                       timeout=300, env=_env(), cwd="/tmp")
    assert r.returncode == 0, r.stderr[-2000:]
    lines = [json.loads(ln) for ln in r.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1                      # rank 0 alone prints
    assert lines[0] == {"launcher_ok": True, "world": 2, "ranks": [0, 1], "nccl_debug": "INFO"}


def test_bench_world_size_mismatch_errors():
    env = _env()
    env.update(WORLD_SIZE="1", RANK="0", LOCAL_RANK="0")
    r = subprocess.run([sys.executable, BENCH, "--gpus", "2", "--selftest-launch"], capture_output=True, text=True,
                       timeout=120, env=env, cwd="/tmp")
    assert r.returncode != 0 and "WORLD_SIZE=1" in (r.stderr + r.stdout)


def test_bench_gpus_2_without_gpus_errors():
    import torch
    if torch.cuda.device_count() >= 2:
        pytest.skip("a 2-GPU box: the launch would run")
    r = subprocess.run([sys.executable, BENCH, "--gpus", "2", "--steps", "1"], capture_output=True, text=True,
                       timeout=300, env=_env(), cwd="/tmp")
    assert r.returncode == 2
    assert "needs 2 visible GPUs" in r.stderr
    assert not [ln for ln in r.stdout.splitlines() if ln.startswith("{")]


def test_cpu_baseline_all_cores_fields():
    code = ("import sys, json; sys.path.insert(0, %r); import bench\n"
            "if __name__ == '__main__':\n"
            "    print(json.dumps(bench.cpu_baseline('j2d5_256_clamp', 0.5, 0.5)))\n") % ROOT
    r = subprocess.run([sys.executable, "-c", code], capture_output=True, text=True, timeout=300, cwd="/tmp")
    assert r.returncode == 0, r.stderr[-2000:]
    d = json.loads(r.stdout.strip().splitlines()[-1])
    assert d["kind"] == "oracle" and d["cores"] == min(os.cpu_count(), 64) and d["nproc"] == os.cpu_count()
    assert d["value"] > 0 and d["single_core_value"] > 0
    assert "cpu_model" in d
