#!/usr/bin/env python
"""Benchmark of the Lift-stencil hot path on B200 (driver contract).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--workload NAME] [--impl reference]

Default workload: BASELINE.json config "Jacobi 3D 7-point, 512^3 fp32, clamp
boundary, 100 time steps" — the config the metric's 1/2/4/8-GPU numbers are
quoted on (north_star: iterated sweeps at 2/4/8 GPUs, weak scaling for the
iterated 3D Jacobi).  One bench step = one full stencil_iterate of 100 time
steps (pad -> slide -> map -> store, iterated) over 512^3 points per GPU.
At N GPUs the global grid is (512*N, 512, 512), slab-decomposed along z; ghost
planes travel by NCCL send/recv overlapped with interior compute, 4 planes
every 4 time steps by default (deep halos, --halo-depth; weak scaling).
`python bench.py --gpus N` launches the N ranks itself through
torch.distributed.run (the driver's launch line) and fails if fewer than N
GPUs are visible.  Inputs (512 MiB per grid) are larger than L2 (126 MB), so
no L2 flush is needed between timed iterations.

Iterated workloads use the plan's AUTO time blocking (--time-block 0): the
7-point weighted star (J3D7) and the 7-point Acoustic update advance two time
steps per pass (K2R / K2RA, bitwise equal to single steps); --time-block 1
forces one step per pass, and the line's "single_step" object reports that
rate and its HBM fraction beside the headline.  roofline.time_steps_per_launch
says how many time steps one launch's algorithmic bytes cover.  "e2e" is the
batched end-to-end call (stencil_run_host_batch: one job per bench step with
its own host->device input copy and device->host result copy, the copies of
neighbouring jobs overlapped with compute).

Other workloads (--workload, stencil_inputs.WORKLOAD_NAMES): the remaining
BASELINE.json configs (gauss5_8192_mirror, j2d5_256_clamp,
hotspot3d_8x512x512[_x100], srad1_4096, srad2_4096, srad_iter_4096,
acoustic7_1024, acoustic13_1024) and the Table-1 workloads (t1_*).
Workloads whose per-sweep bytes are below 2 x L2 are timed cold: a 2 x L2
buffer is written, then another 2 x L2 buffer read, before every timed step
(outside its event pair; L2 then holds clean lines) and a single-sweep
workload's step is one sweep; the warm number is reported as
"hot" (--no-flush times warm).  --scaling strong splits the single-GPU grid
over the ranks (Acoustic 1024^3 over 1/2/4/8 GPUs); --halo fused exchanges
ghosts by peer stores from the boundary kernel instead of NCCL.

Metric: stencil Gpoints/s = output points x time steps / time (PAPER.md
P:958-959 "elements updated per second"); roofline: algorithmic HBM bytes per
launch / average launch time vs MEASURED_PEAKS.json hbm_gbs.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "stencil Gpoints/s & achieved HBM GB/s vs 8 TB/s at 1/2/4/8 B200"

# algorithmic (compulsory) HBM bytes per output point per launch
# SRAD (full iteration): the fused pass reads I, writes I' (8 B) and emits the
# q0 statistics of I' for the next iteration; only the first iteration of a
# stencil_iterate chain reads I once more for its q0 (timed, not counted)
BYTES_PER_POINT = {0: 8, 1: 12, 2: 8, 3: 12, 4: 12, 5: 12, 6: 8, 7: 8}
L2_BYTES = 126e6     # B200 L2 (the flush writes 2x this before each timed step of an L2-resident workload)

def env_int(k, d):
    try:
        return int(os.environ.get(k, d))
    except ValueError:
        return d


def peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        with open(p) as f:
            d = json.load(f)
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    return 6650.0, "fallback (B200_PROFILING.md)"


def ncu_traffic(workload, kernel=None):
    """dram bytes per launch of the dominant kernel from the committed ncu capture
    (the entry "workload:kernel" when the step's kernel has its own capture)."""
    p = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if not os.path.exists(p):
        return None
    with open(p) as f:
        d = json.load(f)
    v = d.get(f"{workload}:{kernel}") if kernel else None
    if v is None:
        v = d.get(workload)
        if v is not None and kernel and kernel not in v.get("kernel", kernel):
            return None          # the capture is of another kernel
    return None if v is None else v.get("dram_bytes_per_launch")


class ClockSampler:
    """SM clock + throttle reasons sampled during the timed region.

    NVML (the library nvidia-smi reads) every 20 ms, so even a ~1 s timed
    region gets dozens of samples; falls back to nvidia-smi if NVML is absent."""

    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
         "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")

    def __init__(self, gpu_index):
        self.idx = gpu_index
        self.samples = []
        self.stop = threading.Event()
        self.t = threading.Thread(target=self.run, daemon=True)
        # NVML is initialised here, before the timed region (nvmlInit can take
        # longer than a short timed region: the sampler thread would start late)
        self.nv = self.h = None
        try:
            import pynvml as nv
            nv.nvmlInit()
            vis = os.environ.get("CUDA_VISIBLE_DEVICES")
            idx = int(vis.split(",")[self.idx]) if vis and vis.split(",")[self.idx].isdigit() else self.idx
            self.h = nv.nvmlDeviceGetHandleByIndex(idx)
            self.mx = nv.nvmlDeviceGetMaxClockInfo(self.h, nv.NVML_CLOCK_SM)
            self.nv = nv
        except Exception:
            self.nv = None

    def sample_nvml(self):
        nv, h = self.nv, self.h
        bits = [0x8, 0x40, 0x20, 0x4]    # hw_slowdown, hw_thermal, sw_thermal, sw_power_cap
        sm = nv.nvmlDeviceGetClockInfo(h, nv.NVML_CLOCK_SM)
        rs = nv.nvmlDeviceGetCurrentClocksEventReasons(h)
        self.samples.append([str(sm), str(self.mx)] + ["Active" if rs & b else "Not Active" for b in bits])

    def run(self):
        if self.nv is not None:
            try:
                while not self.stop.is_set():
                    self.sample_nvml()
                    self.stop.wait(0.02)
                return
            except Exception:
                pass
        while not self.stop.is_set():
            try:
                r = subprocess.run(["nvidia-smi", "-i", str(self.idx), f"--query-gpu={self.Q}",
                                    "--format=csv,noheader,nounits"], capture_output=True, text=True, timeout=5)
                vals = [v.strip() for v in r.stdout.strip().split(",")]
                if len(vals) == 6:
                    self.samples.append(vals)
            except Exception:
                pass
            self.stop.wait(0.2)

    def __enter__(self):
        self.t.start()
        return self

    def __exit__(self, *a):
        # one more sample at the end of the timed region (before the sync's
        # return lets the clocks drop), then stop
        if self.nv is not None:
            try:
                self.sample_nvml()
            except Exception:
                pass
        self.stop.set()
        self.t.join(timeout=10)
        if self.nv is not None:
            try:
                self.nv.nvmlShutdown()
            except Exception:
                pass

    def summary(self):
        if not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"], "samples": 0}
        sm = [float(s[0]) for s in self.samples if s[0].replace(".", "").isdigit()]
        mx = [float(s[1]) for s in self.samples if s[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for s in self.samples for i in range(4) if s[2 + i].lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": reasons, "samples": len(self.samples)}


# ----------------------------------------------------------------------------
# reference arm / cpu baseline: the fp64 oracle on a bounded sample
# ----------------------------------------------------------------------------
def oracle_sample_spec(workload):
    """A bounded sub-grid of the workload (same op/kind/weights), ~seconds of CPU."""
    import stencil_inputs as si
    w = si.workload(workload)
    ext = w.spec.extents
    if len(ext) == 3:
        sub = (min(ext[0], 16), min(ext[1], 512), min(ext[2], 512))
    else:
        sub = (min(ext[0], 1024), min(ext[1], 1024))
    ws = si.workload(workload, scale=sub)
    xs, spec = si.make_workload_inputs(ws)
    return xs, spec, sub


def time_oracle(workload, min_seconds=10.0, max_reps=50):
    """The oracle on ONE core: repeated sweeps of the bounded sub-grid."""
    from oracle import stencil_oracle as orc
    xs, spec, sub = oracle_sample_spec(workload)
    pts = int(np.prod(spec.out_extents()))
    reps = 0
    t0 = time.perf_counter()
    while True:
        orc.apply(spec, xs)
        reps += 1
        el = time.perf_counter() - t0
        if el >= min_seconds or reps >= max_reps:
            break
    gpts = pts * reps / el / 1e9
    sample = f"{reps} x one sweep of a {'x'.join(map(str, sub))} sub-grid of {workload} (numpy fp64 oracle)"
    return gpts, sample, el


def _oracle_worker_init():
    # one single-threaded numpy per process (no BLAS / OpenMP threads)
    for k in ("OMP_NUM_THREADS", "OPENBLAS_NUM_THREADS", "MKL_NUM_THREADS"):
        os.environ[k] = "1"


def _oracle_worker(task):
    """One process of the all-core oracle run: ``reps`` sweeps of its own
    sub-grid (an independent z-slab sample of the workload, seeded by its
    index).  Returns (points computed, seconds)."""
    workload, idx, reps = task
    import stencil_inputs as si
    from oracle import stencil_oracle as orc
    xs, spec, sub = oracle_sample_spec(workload)
    if idx:
        xs = [np.roll(x, idx, axis=-1) for x in xs]     # a different slab's values, same shape and op
    pts = int(np.prod(spec.out_extents()))
    t0 = time.perf_counter()
    for _ in range(reps):
        orc.apply(spec, xs)
    return pts * reps, time.perf_counter() - t0


def cpu_model():
    try:
        out = subprocess.run(["lscpu"], capture_output=True, text=True, timeout=10).stdout
        for ln in out.splitlines():
            if ln.startswith("Model name:"):
                return ln.split(":", 1)[1].strip()
    except Exception:
        pass
    return None


class OraclePool:
    """The oracle on all host cores: one single-threaded process per core, each
    sweeping its own bounded sub-grid of the workload (the work is
    embarrassingly parallel over z-slabs, as the slab decomposition is)."""

    def __init__(self, workload, max_procs=64):
        import multiprocessing as mp
        self.workload = workload
        self.nproc = os.cpu_count() or 1
        self.procs = max(1, min(self.nproc, max_procs))
        self.pool = mp.get_context("spawn").Pool(self.procs, initializer=_oracle_worker_init)
        # warm-up: every worker imports numpy/oracle and builds its inputs once
        self.pool.map(_oracle_worker, [(workload, i, 0) for i in range(self.procs)])

    def run(self, reps):
        t0 = time.perf_counter()
        res = self.pool.map(_oracle_worker, [(self.workload, i, reps) for i in range(self.procs)])
        el = time.perf_counter() - t0
        pts = sum(r[0] for r in res)
        return pts / el / 1e9, el

    def close(self):
        self.pool.close()
        self.pool.join()


def cpu_baseline(workload, single_seconds=8.0, all_seconds=8.0):
    """Oracle timed on one core and on all host cores (rank 0, N=1)."""
    g1, sample1, el1 = time_oracle(workload, min_seconds=single_seconds, max_reps=20)
    xs, spec, sub = oracle_sample_spec(workload)
    per_rep = int(np.prod(spec.out_extents())) / (g1 * 1e9)      # seconds per sweep on one core
    pool = OraclePool(workload)
    try:
        reps = max(1, int(all_seconds / max(per_rep, 1e-3)))
        gall, elall = pool.run(reps)
    finally:
        pool.close()
    return {"value": gall, "unit": "Gpoints/s", "cores": pool.procs, "nproc": pool.nproc, "kind": "oracle",
            "cpu_model": cpu_model(),
            "sample": f"{pool.procs} processes x {reps} sweeps of a {'x'.join(map(str, sub))} sub-grid of "
                      f"{workload} each (numpy fp64 oracle, one single-threaded process per core)",
            "single_core_value": g1, "single_core_sample": sample1}


def reference_arm(args, workload):
    rank = env_int("RANK", 0)
    if rank != 0:
        return
    # each step: one sweep of the bounded sub-grid in every process of the
    # all-core oracle pool (one single-threaded process per host core)
    pool = OraclePool(workload)
    try:
        for _ in range(args.warmup):
            pool.run(1)
        per_step, gp_all = [], []
        for _ in range(args.steps):
            gp, el = pool.run(1)
            gp_all.append(gp)
            per_step.append(el)
    finally:
        pool.close()
    gpts = statistics.median(gp_all)
    xs, spec, sub = oracle_sample_spec(workload)
    sample = (f"per step: {pool.procs} processes x one sweep of a {'x'.join(map(str, sub))} sub-grid of "
              f"{workload} (numpy fp64 oracle, one single-threaded process per core)")
    line = {"impl": "reference", "metric": METRIC, "value": gpts, "unit": "Gpoints/s", "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": 1e3 * statistics.median(per_step),
            "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
            "config": {"workload": workload},
            "cpu_baseline": {"value": gpts, "unit": "Gpoints/s", "cores": pool.procs, "nproc": pool.nproc,
                             "cpu_model": cpu_model(), "kind": "oracle", "sample": sample},
            "e2e": {"value": gpts, "unit": "Gpoints/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


class HostStagedExchange:
    """Test transport (--test-transport staged): the slab's ghost exchange with
    DistExchange's neighbour pairing, the planes staged through host memory
    over gloo (ranks sharing one GPU cannot use NCCL)."""

    def __init__(self, rank, world, n, g, wrap, group=None):
        from paper_conf_cgo_hagedornssgd18_b200.slab import DistExchange
        self.inner = DistExchange(rank, world, n, g, wrap, group)

    def post(self, buf):
        import torch
        import torch.distributed as dist
        ex = self.inner
        n, g = ex.n, ex.g
        if ex.self_wrap or (ex.lo is None and ex.hi is None):
            return ex.post(buf)
        low, high = buf[g:2 * g].cpu(), buf[n:n + g].cpu()
        rlo, rhi = torch.empty_like(low), torch.empty_like(high)
        ops = []
        if ex.lo is not None:
            ops.append(dist.P2POp(dist.isend, low, ex.lo, tag=0))
        if ex.hi is not None:
            ops.append(dist.P2POp(dist.irecv, rhi, ex.hi, tag=0))
        if ex.hi is not None:
            ops.append(dist.P2POp(dist.isend, high, ex.hi, tag=1))
        if ex.lo is not None:
            ops.append(dist.P2POp(dist.irecv, rlo, ex.lo, tag=1))
        for w in dist.batch_isend_irecv(ops):
            w.wait()
        if ex.lo is not None:
            buf[0:g].copy_(rlo)
        if ex.hi is not None:
            buf[n + g:n + 2 * g].copy_(rhi)
        return []


# ----------------------------------------------------------------------------
# launcher: --gpus N without torchrun re-executes through torch.distributed.run
# ----------------------------------------------------------------------------
def _free_port():
    import socket
    with socket.socket(socket.AF_INET, socket.SOCK_STREAM) as so:
        so.bind(("127.0.0.1", 0))
        return so.getsockname()[1]


def launch_ranks(nprocs, argv):
    """One process per GPU: ``python -m torch.distributed.run --nnodes=1
    --nproc-per-node N --master-addr 127.0.0.1 --master-port P bench.py ...``
    (the driver's own launch line).  NCCL_DEBUG=INFO unless set, written to
    stderr, so the communicator's nranks shows in the log while stdout keeps
    the one JSON line.  Returns the exit code."""
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={nprocs}",
           "--master-addr", "127.0.0.1", "--master-port", str(_free_port()), os.path.abspath(__file__)] + list(argv)
    env = dict(os.environ)
    env.setdefault("NCCL_DEBUG", "INFO")
    env.setdefault("NCCL_DEBUG_FILE", "/dev/stderr")    # keep stdout to the one JSON line
    return subprocess.call(cmd, env=env)


def launcher_selftest(args):
    """--selftest-launch: each rank joins a gloo group and checks that the
    world is exactly --gpus ranks (CPU test of the launcher path)."""
    import torch
    import torch.distributed as dist
    world = env_int("WORLD_SIZE", 1)
    if world != args.gpus:
        raise SystemExit(f"bench.py: --gpus {args.gpus} but WORLD_SIZE={world}")
    if world > 1:
        dist.init_process_group("gloo")
        assert dist.get_world_size() == args.gpus
        t = torch.tensor([dist.get_rank()], dtype=torch.int64)
        ranks = [torch.zeros_like(t) for _ in range(world)]
        dist.all_gather(ranks, t)
        ranks = [int(r.item()) for r in ranks]
        dist.destroy_process_group()
    else:
        ranks = [0]
    if env_int("RANK", 0) == 0:
        print(json.dumps({"launcher_ok": True, "world": world, "ranks": ranks,
                          "nccl_debug": os.environ.get("NCCL_DEBUG")}), flush=True)


# ----------------------------------------------------------------------------
# CUDA arm
# ----------------------------------------------------------------------------
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--workload", default="j3d7_512_clamp")
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--no-flush", action="store_true",
                    help="L2-resident workloads: time L2-warm back-to-back sweeps instead of cold flushed steps")
    ap.add_argument("--no-graph", action="store_true", help="launch single sweeps eagerly instead of a CUDA graph")
    ap.add_argument("--time-block", type=int, default=0, choices=[0, 1, 2],
                    help="iterate time steps per pass: 0 = AUTO (two where the register two-step kernel K2R "
                         "applies), 1 = single steps, 2 = two steps where K2R/K2T apply")
    ap.add_argument("--scaling", default="weak", choices=["weak", "strong"],
                    help="multi-GPU iterated sweeps: weak = the single-GPU grid per rank (default), "
                         "strong = the single-GPU grid split over the ranks")
    ap.add_argument("--force-slab", action="store_true",
                    help="run the slab (multi-GPU) path even at world size 1 (launch under torchrun)")
    ap.add_argument("--halo", default="nccl", choices=["nccl", "fused"],
                    help="multi-GPU ghost exchange: NCCL send/recv overlapped with the interior (default), or the "
                         "fused boundary kernel storing into the neighbours' ghosts over NVLink peer memory")
    ap.add_argument("--halo-depth", type=int, default=None,
                    help="slab path: ghost depth in time steps k (NEXT-3 deep halos): ghosts of r*k planes are "
                         "exchanged every k time steps and the overlap is recomputed redundantly (default 4 on "
                         "the NCCL path: 797 vs 750 Gpts/s at world size 1, profiles/r02_slab_world1.txt; the "
                         "fused path exchanges every step)")
    ap.add_argument("--selftest-launch", action="store_true", help=argparse.SUPPRESS)
    # test-only transport: N ranks share cuda:0 over gloo, ghost planes staged
    # through host memory (NCCL refuses two ranks on one GPU) — exercises the
    # whole multi-rank bench path (partition, exchange schedule, timing, the
    # JSON line) on a one-GPU box
    ap.add_argument("--test-transport", default=None, choices=["staged"], help=argparse.SUPPRESS)
    args = ap.parse_args()
    args.warmup = max(args.warmup, 3)
    if args.halo_depth is None:
        args.halo_depth = 1 if args.halo == "fused" else 4

    # --gpus N without a torchrun environment: launch N ranks ourselves (the
    # same launch line the driver uses), so `python bench.py --gpus N` is a
    # real N-process run; N = 1 runs in this process (the same code path)
    if args.gpus > 1 and "WORLD_SIZE" not in os.environ and args.impl == "ours":
        if not args.selftest_launch and not args.test_transport:
            import torch
            have = torch.cuda.device_count()
            if have < args.gpus:
                print(f"bench.py: --gpus {args.gpus} needs {args.gpus} visible GPUs, found {have}", file=sys.stderr)
                sys.exit(2)
        sys.exit(launch_ranks(args.gpus, sys.argv[1:]))
    if args.selftest_launch:
        launcher_selftest(args)
        return

    if args.impl == "reference":
        reference_arm(args, args.workload)
        return

    import torch
    import torch.distributed as dist

    import stencil_inputs as si
    import paper_conf_cgo_hagedornssgd18_b200 as lift
    from paper_conf_cgo_hagedornssgd18_b200.slab import SlabPlan, symmetric_fused_halo

    world = env_int("WORLD_SIZE", 1)
    sym, fused = None, None
    rank = env_int("RANK", 0)
    local = env_int("LOCAL_RANK", 0)
    staged = args.test_transport == "staged"
    if staged:
        local = 0                                   # every rank on cuda:0 (test transport)
        if args.halo == "fused":
            raise SystemExit("bench.py: the staged test transport exchanges through host memory (no --halo fused)")
    if world != args.gpus:
        raise SystemExit(f"bench.py: --gpus {args.gpus} but the launch has WORLD_SIZE={world} ranks")
    if torch.cuda.device_count() <= local:
        raise SystemExit(f"bench.py: rank {rank} needs cuda:{local}, {torch.cuda.device_count()} GPUs visible")
    torch.cuda.set_device(local)
    use_pg = world > 1 or (args.force_slab and "MASTER_ADDR" in os.environ)
    if use_pg:
        if staged:
            dist.init_process_group("gloo")
        else:
            os.environ.setdefault("NCCL_DEBUG", "INFO")        # communicator nranks in the log (stderr)
            os.environ.setdefault("NCCL_DEBUG_FILE", "/dev/stderr")
            dist.init_process_group("nccl", device_id=torch.device(f"cuda:{local}"))
        if dist.get_world_size() != args.gpus:
            raise SystemExit(f"bench.py: process group has {dist.get_world_size()} ranks, --gpus {args.gpus}")

    def max_over_ranks(v: float) -> float:
        if not use_pg:
            return v
        tt = torch.tensor([v], dtype=torch.float64, device="cpu" if staged else dev)
        dist.all_reduce(tt, op=dist.ReduceOp.MAX)
        return float(tt.item())
    dev = torch.device(f"cuda:{local}")

    w = si.workload(args.workload)
    steps_per_iter = w.steps
    spec = w.spec
    ext1 = spec.extents
    iterable = spec.op in (si.WEIGHTED, si.HOTSPOT3D, si.ACOUSTIC, si.SRAD) and steps_per_iter > 1
    slabbed = (world > 1 or (args.force_slab and use_pg)) and iterable and len(ext1) == 3

    # ---- inputs: seeded synthetic grids resident in HBM (host copies kept for e2e)
    local_ext = ext1
    if slabbed:
        from paper_conf_cgo_hagedornssgd18_b200.slab import partition
        ws = si.workload(args.workload)
        if args.scaling == "weak":
            # weak scaling: the per-rank slab is the single-GPU workload
            gext = (ext1[0] * world,) + tuple(ext1[1:])
            ws.spec.extents = ext1
        else:
            # strong scaling: the single-GPU grid is split over the ranks
            gext = tuple(ext1)
            z0, z1 = partition(ext1[0], world)[rank]
            ws.spec.extents = (z1 - z0,) + tuple(ext1[1:])
        seeds = tuple(s + 7919 * rank for s in ws.seeds)
        ws.seeds = seeds
        xs, spec = si.make_workload_inputs(ws)
    else:
        ws = si.workload(args.workload)
        ws.seeds = tuple(s + 7919 * rank for s in ws.seeds)
        xs, spec = si.make_workload_inputs(ws)
    npts_local = int(np.prod(spec.out_extents()))

    if slabbed:
        sp = SlabPlan(gext, rank, world, spec.size, spec.pad_lo, list(spec.kind), spec.pad_value, spec.op,
                      spec.weights, spec.params, device=local, depth=args.halo_depth,
                      exchange_factory=HostStagedExchange if staged else None)
        plan = sp.plan
        host = [torch.from_numpy(x).pin_memory() for x in xs]
        bufs = []
        fused = None
        if args.halo == "fused":
            sym, fused = symmetric_fused_halo(sp)
        for i, x in enumerate(host):
            # the rotating state lives in symmetric (peer-mapped) memory for the fused path
            is_state = i == 0 or spec.op == si.ACOUSTIC
            b = sym[i] if (fused is not None and is_state) else sp.empty()
            sp.owned(b).copy_(x, non_blocking=True)
            bufs.append(b)
    else:
        plan = lift.Plan.from_spec(spec, device=local)
        plan.set_time_block(args.time_block)
        host = [torch.from_numpy(x).pin_memory() for x in xs]
        bufs = [x.to(dev, non_blocking=True) for x in host]
    torch.cuda.synchronize()
    if use_pg:
        # a collective first: NCCL point-to-point batches then run on an
        # initialised communicator (torch's batch_isend_irecv requirement)
        dist.barrier()

    # state/aux layout per op
    op = spec.op
    if iterable:
        if op == si.ACOUSTIC:
            state = [bufs[0], bufs[1]]          # prev, cur
            if not slabbed and args.time_block != 1:
                # two spare grids: two steps per pass where K2RA applies
                state += [torch.empty_like(bufs[0]), torch.empty_like(bufs[0])]
            aux = []
        elif op == si.HOTSPOT3D:
            state = [bufs[0], sym[1] if (slabbed and fused is not None) else torch.empty_like(bufs[0])]
            aux = [bufs[1]]
        else:
            state = [bufs[0], sym[1] if (slabbed and fused is not None) else torch.empty_like(bufs[0])]
            aux = []
        # slab + NCCL: boundary low, boundary high, interior per time step;
        # slab + fused: one launch per time step
        launches_per_step = steps_per_iter
        if slabbed and args.halo == "nccl":
            # every block of k steps: k - 1 extended sweeps, then boundary low,
            # boundary high and interior of its last step; with two-step passes
            # (weighted 7-point star, ghosts >= 2: slab.deep_halo_iterate) the
            # block's steps run in pairs, an odd block starting with one step
            two = op == si.WEIGHTED and sp.plan.time_block == 2 and sp.r == 1
            launches_per_step = 0
            left = steps_per_iter
            while left > 0:
                kb = min(args.halo_depth, left)
                if two and kb >= 2:
                    launches_per_step += (kb % 2) + (kb // 2 - 1) + 3
                else:
                    launches_per_step += kb + 2
                left -= kb
        if op == si.SRAD:
            launches_per_step = steps_per_iter + 1        # q0 partials of the input, then one fused pass per iteration
    else:
        out = plan.empty_output()
        launches_per_step = 1
    tb = plan.time_block if (iterable and not slabbed) else 1     # time steps per launch (K2R / K2T: 2)
    if tb == 2:
        launches_per_step = steps_per_iter // 2 + steps_per_iter % 2
    # a bench step of a single-sweep workload is a CUDA graph of `sweeps` full
    # sweeps (each reads the whole input and writes the whole output): small
    # grids (J2D5 256^2) take microseconds per sweep, so one graph launch per
    # sweep would time the host, not the kernel
    sweeps = 1 if iterable else int(min(1000, max(1, (1 << 26) // max(1, npts_local))))
    launches_per_step *= sweeps

    stream = torch.cuda.current_stream()

    def step():
        if iterable:
            if slabbed:
                return sp.iterate(state, steps_per_iter, aux, fused=fused)
            return plan.iterate(state, steps_per_iter, aux)
        for _ in range(sweeps):
            plan.apply(*bufs, out=out)
        return 0

    # single-GPU steps are captured once into a CUDA graph (the C-ABI calls are
    # graph-capturable by design: stream-ordered, no allocation, no sync) and
    # replayed; the slab path keeps its stream launches (NCCL + side streams)
    graph = None
    if not slabbed and not args.no_graph:
        side = torch.cuda.Stream()
        side.wait_stream(torch.cuda.current_stream())
        with torch.cuda.stream(side):
            step()
        torch.cuda.current_stream().wait_stream(side)
        graph = torch.cuda.CUDAGraph()
        with torch.cuda.graph(graph):
            step()
        eager_step = step

        def step():  # noqa: F811
            graph.replay()
            return 0

    def barrier():
        if use_pg:
            dist.barrier()
        torch.cuda.synchronize()

    # warm-up
    for _ in range(args.warmup):
        step()
    barrier()
    # K4 / K6 (persistent iterate of a small 3D grid): one launch per bench step
    persist = (not slabbed) and iterable and plan.last_variant in (3, 5)
    if persist:
        launches_per_step = 1
    variant_id = plan.last_variant if persist else plan.variant

    # L2-resident working sets (one sweep's algorithmic bytes < 2 x L2): the
    # timed steps are cold — a 2 x L2 buffer is written before every step,
    # outside the step's event pair — and single-sweep workloads time ONE
    # sweep per step; the hot number (graph of back-to-back sweeps, L2-warm)
    # is reported beside it as "hot"
    bpp = BYTES_PER_POINT[op]
    # algorithmic bytes of one launch: a two-step Acoustic pass (K2RA) reads
    # u^{n-1}, u^n and writes u^{n+1}, u^{n+2}; a two-step weighted pass (K2R)
    # reads X_t and writes X_{t+2}
    bpp_launch = 16 if (tb == 2 and op == si.ACOUSTIC) else bpp
    cold = (not slabbed) and npts_local * bpp < 2 * L2_BYTES and not args.no_flush
    hot = None
    if cold:
        def time_hot():
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            barrier()
            e0.record(stream)
            for _ in range(args.steps):
                step()
            e1.record(stream)
            barrier()
            th = e0.elapsed_time(e1)
            return {"value": npts_local * steps_per_iter * sweeps * args.steps / (th * 1e-3) / 1e9,
                    "sweeps_per_step": steps_per_iter if iterable else sweeps,
                    "ms_per_step": th / args.steps, "l2": "warm (back-to-back sweeps, no flush)"}
        hot = time_hot()
        # the flush writes 2 x L2, then reads another 2 x L2 buffer: the write
        # evicts the working set, the read leaves L2 holding CLEAN lines, so
        # the timed sweep does not pay for writing back the flush buffer's
        # dirty lines (measured: +2-3 us per cold sweep of an 8 MB grid,
        # profiles/r02_latency_probe.txt) — the state ncu's cache control gives
        flush = torch.empty(int(2 * L2_BYTES) // 4, dtype=torch.int32, device=dev)
        flush_rd = torch.ones(int(2 * L2_BYTES) // 4, dtype=torch.int32, device=dev)
        flush_sink = torch.empty((), dtype=torch.int64, device=dev)
        if not iterable:
            one = None
            if graph is not None:
                one = torch.cuda.CUDAGraph()
                side = torch.cuda.Stream()
                side.wait_stream(torch.cuda.current_stream())
                with torch.cuda.stream(side):
                    plan.apply(*bufs, out=out)
                torch.cuda.current_stream().wait_stream(side)
                with torch.cuda.graph(one):
                    plan.apply(*bufs, out=out)

            def step():  # noqa: F811  (one cold sweep)
                if one is not None:
                    one.replay()
                else:
                    plan.apply(*bufs, out=out)
                return 0
            launches_per_step //= sweeps
            sweeps = 1
            for _ in range(2):
                step()
    # timed region: exactly K steps, barrier + sync on both sides, events on the launching stream
    ev0 = torch.cuda.Event(enable_timing=True)
    ev1 = torch.cuda.Event(enable_timing=True)
    with ClockSampler(local) as clk:
        barrier()
        if cold:
            pairs = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True))
                     for _ in range(args.steps)]
            for k in range(args.steps):
                flush.fill_(k)              # evict the working set from L2 (not timed)
                torch.sum(flush_rd, 0, out=flush_sink)   # ... and leave clean lines behind
                pairs[k][0].record(stream)
                step()
                pairs[k][1].record(stream)
        else:
            ev0.record(stream)
            for _ in range(args.steps):
                step()
            ev1.record(stream)
        barrier()
    t_ms = sum(a.elapsed_time(b) for a, b in pairs) if cold else ev0.elapsed_time(ev1)
    t_max = max_over_ranks(t_ms)
    ms_per_step = t_max / args.steps
    points = npts_local * world * steps_per_iter * sweeps * args.steps
    value = points / (t_max * 1e-3) / 1e9

    # per-launch kernel duration of the dominant kernel: a step is back-to-back
    # launches of it on one stream (single GPU), so avg launch = step time / launches
    if not slabbed:
        # the step is back-to-back launches of the dominant kernel on one stream
        # (SRAD: one iteration = one fused pass; the first iteration's q0 pass is in the time)
        units = args.steps * (steps_per_iter if op == si.SRAD else launches_per_step)
        if persist:   # K4 / K6: one launch per bench step runs all time steps; time per time step
            units = args.steps * steps_per_iter
        avg_launch_s = (t_ms * 1e-3) / units
        alg_bytes = npts_local * bpp_launch
    else:
        # time the owned-slab sweep alone (all planes in one launch) on this rank
        e0 = torch.cuda.Event(enable_timing=True)
        e1 = torch.cuda.Event(enable_timing=True)
        nrep = 20
        ins = (state[0],) + tuple(aux) if op != si.ACOUSTIC else (state[0], state[1])
        dst = state[1] if op != si.ACOUSTIC else state[0]
        # the kernel the slab step runs: two-step passes (K2R) inside the
        # deep-halo blocks of a weighted 7-point star, else single sweeps
        two_slab = op == si.WEIGHTED and args.halo == "nccl" and args.halo_depth >= 2 and \
            sp.plan.time_block == 2 and sp.r == 1

        def owned():
            if two_slab:
                plan.apply2_region(state[0], out=state[1], begin=0, end=sp.n)
            else:
                plan.apply(*ins, out=dst)
        owned()                                   # (first launch of this kernel in the process: module load)
        torch.cuda.synchronize()
        e0.record(stream)
        for _ in range(nrep):
            owned()
        e1.record(stream)
        torch.cuda.synchronize()
        avg_launch_s = e0.elapsed_time(e1) * 1e-3 / nrep
        alg_bytes = npts_local * bpp
        if two_slab:
            tb = 2
    peak, peak_src = peaks()
    achieved = alg_bytes / avg_launch_s / 1e9
    kernel_name = plan.last_kernel          # the kernel function the timed step launched (stencil_plan_last_kernel)

    # ---- halo exchange (slab path): bytes per rank, exchange time, NVLink fraction
    halo = None
    if slabbed:
        from paper_conf_cgo_hagedornssgd18_b200.slab import neighbours
        lo_nb, hi_nb = neighbours(rank, world, sp.wrap)
        n_nb = (lo_nb is not None) + (hi_nb is not None)
        plane_bytes = int(np.prod(spec.extents[1:])) * 4
        k = args.halo_depth
        grids = 2 if (op == si.ACOUSTIC and k > 1) else 1      # grids exchanged per exchange
        per_nb = sp.g * plane_bytes * grids                     # bytes to (and from) each neighbour per exchange
        exchanges_per_step = -(-steps_per_iter // k) if args.halo == "nccl" else steps_per_iter
        ex_us = None
        if args.halo == "nccl" and world > 1:
            # the exchange alone (no compute), posted like in the step, max over ranks
            exb = [state[0]] + ([state[1]] if grids == 2 else [])
            nrep = 20
            x0, x1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            barrier()
            x0.record(stream)
            for _ in range(nrep):
                sp._join(sp._on_comm(lambda: sp._post(exb)))
            x1.record(stream)
            barrier()
            ex_us = max_over_ranks(x0.elapsed_time(x1) / nrep) * 1e3
        nvl_gbs = per_nb / (ex_us * 1e-6) / 1e9 if ex_us else None
        halo = {"path": args.halo, "depth_steps": k, "ghost_planes": sp.g, "grids_per_exchange": grids,
                "neighbours": n_nb, "bytes_per_neighbour_per_exchange": per_nb,
                "bytes_per_rank_per_time_step": per_nb * n_nb * exchanges_per_step / steps_per_iter,
                "exchanges_per_bench_step": exchanges_per_step,
                "exchanges_per_100_time_steps": -(-100 // k) if args.halo == "nccl" else 100,
                "exchange_us": ex_us,
                "nvlink_gbs_per_direction": nvl_gbs,
                "nvlink_peak_gbs_per_direction": 900.0,
                "nvlink_frac": (nvl_gbs / 900.0) if nvl_gbs else None,
                "exchange_share_of_time_step": ((ex_us * 1e-3) * exchanges_per_step / ms_per_step) if ex_us else None,
                "owned_sweep_gpts": npts_local * tb / avg_launch_s / 1e9,
                "owned_sweep_time_steps_per_launch": tb}

    # ---- e2e: the C-ABI call with HOST buffers (H2D + compute + D2H timed), single GPU path
    e2e = None
    if not args.no_e2e and not slabbed:
        h_state = [x.numpy() for x in host]
        h_aux = []
        if op == si.HOTSPOT3D:                   # T is the state, P the fixed aux grid
            h_state, h_aux = [host[0].numpy()], [host[1].numpy()]
        outs_h = [torch.empty(plan.out_alloc_extents, dtype=torch.float32).pin_memory().numpy() for _ in range(2)]
        nsteps = steps_per_iter if iterable else 1
        # one bench step = one job of stencil_run_host_batch: its own H2D of the
        # inputs from pinned host memory, the iterate, the D2H of its result;
        # the batch overlaps job j+1's H2D and job j-1's D2H with job j's compute
        n_e2e = max(2, min(args.steps, 10))
        jobs = [h_state] * n_e2e
        aux_jobs = [h_aux] * n_e2e if h_aux else ()
        outs = [outs_h[j % 2] for j in range(n_e2e)]
        plan.run_host_batch(jobs[:2], nsteps, aux_jobs[:2] if h_aux else (), outs[:2])   # warm (workspace)
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        plan.run_host_batch(jobs, nsteps, aux_jobs, outs)
        el = (time.perf_counter() - t0) / n_e2e
        h2d = sum(a.nbytes for a in h_state) + sum(a.nbytes for a in h_aux)
        # the single-job call, for reference (no overlap: H2D, compute, D2H in sequence)
        plan.run_host(h_state, nsteps, h_aux, out=outs_h[0])             # warm (its own workspace)
        t1 = time.perf_counter()
        plan.run_host(h_state, nsteps, h_aux, out=outs_h[0])
        el1 = time.perf_counter() - t1
        e2e = {"value": npts_local * nsteps / el / 1e9, "unit": "Gpoints/s", "h2d_bytes_per_step": int(h2d),
               "d2h_bytes_per_step": int(outs_h[0].nbytes), "ms_per_step": el * 1e3,
               "jobs": n_e2e, "single_job_value": npts_local * nsteps / el1 / 1e9,
               "timing": "host wall clock around one stencil_run_host_batch call of `jobs` jobs (synchronising), "
                         "per job; single_job_value: one stencil_run_host call"}
    elif not args.no_e2e and slabbed:
        # per rank: H2D of the owned slab(s) from pinned host memory, the slab
        # iterate (with its halo exchange), D2H of the newest owned grid
        n_e2e = max(1, min(args.steps, 3))
        res_h = torch.empty(sp.owned(state[0]).shape, dtype=torch.float32).pin_memory()
        def e2e_step():
            for b, x in zip(bufs, host):
                sp.owned(b).copy_(x, non_blocking=True)
            ri = sp.iterate(state, steps_per_iter, aux, fused=fused)
            res_h.copy_(sp.owned(state[ri]), non_blocking=True)
        e2e_step()
        barrier()
        q0 = torch.cuda.Event(enable_timing=True)
        q1 = torch.cuda.Event(enable_timing=True)
        q0.record(stream)
        for _ in range(n_e2e):
            e2e_step()
        q1.record(stream)
        barrier()
        te = max_over_ranks(q0.elapsed_time(q1)) / n_e2e
        h2d = sum(int(x.numel()) * 4 for x in host)
        e2e = {"value": npts_local * world * steps_per_iter / (te * 1e-3) / 1e9, "unit": "Gpoints/s",
               "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": int(res_h.numel()) * 4, "ms_per_step": te,
               "timing": "CUDA events, max over ranks, pinned host buffers"}

    # ---- the same workload with one step per pass (temporal
    # blocking raises Gpts/s above the per-sweep HBM roofline, so the per-sweep
    # rate and its bandwidth fraction are reported beside it)
    single_step = None
    if tb == 2 and not slabbed and iterable:
        p1 = lift.Plan.from_spec(spec, device=local)
        p1.set_time_block(1)
        st1 = [torch.empty_like(x) for x in state]
        for a_, b_ in zip(st1, state):
            a_.copy_(b_)

        def step1():
            return p1.iterate(st1, steps_per_iter, aux)
        side = torch.cuda.Stream()
        side.wait_stream(torch.cuda.current_stream())
        with torch.cuda.stream(side):
            step1()
        torch.cuda.current_stream().wait_stream(side)
        g1 = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g1):
            step1()
        for _ in range(max(1, args.warmup)):
            g1.replay()
        torch.cuda.synchronize()
        f0, f1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        f0.record(stream)
        for _ in range(args.steps):
            g1.replay()
        f1.record(stream)
        torch.cuda.synchronize()
        t1_ms = f0.elapsed_time(f1)
        launch1 = t1_ms * 1e-3 / (args.steps * steps_per_iter)
        single_step = {"value": npts_local * steps_per_iter * args.steps / (t1_ms * 1e-3) / 1e9,
                       "ms_per_step": t1_ms / args.steps, "kernel": p1.last_kernel,
                       "roofline_frac": npts_local * bpp / launch1 / 1e9 / peak,
                       "avg_launch_us": launch1 * 1e6}
        del st1, g1

    # ---- cpu baseline: the oracle on a bounded sample (rank 0, N=1 only)
    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu:
        cpu = cpu_baseline(args.workload)

    clocks = clk.summary()
    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": "Gpoints/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms_per_step, "higher_is_better": True,
            "scaling": args.scaling if slabbed else "weak",
            "vs_baseline": None, "dtype": "f32", "data": "synthetic",
            "config": {"workload": args.workload, "extents_per_gpu": list(spec.extents),
                       "global_extents": list(gext) if slabbed else list(ext1),
                       "time_steps_per_bench_step": steps_per_iter if iterable else 1,
                       "time_steps_per_pass": tb,
                       "sweeps_per_bench_step": steps_per_iter if iterable else sweeps,
                       "op": si.OP_NAMES[op], "boundary": [si.KIND_NAMES[k] for k in spec.kind],
                       "window": list(spec.size),
                       "halo": (args.halo if slabbed else None),
                       "halo_depth": (args.halo_depth if slabbed else None),
                       "parallelism": f"slab-z x{world}" if slabbed else
                       (f"replicas x{world}" if world > 1 else "single"),
                       "l2": ("L2 flushed (2 x L2 write, then 2 x L2 read: clean lines) before every timed "
                              "step; one sweep per step"
                              if cold and not iterable else
                              "L2 flushed (2 x L2 write, then 2 x L2 read: clean lines) before every timed step"
                              if cold else
                              "inputs larger than L2 (no flush needed)" if npts_local * bpp >= 2 * L2_BYTES
                              else "L2-resident working set, not flushed (--no-flush)"),
                       "variant": {0: "K0 generic",
                                   1: ("K1 tile2d (TMA)" if ext1[-1] % 4 == 0 else
                                       "K1 tile2d (cp.async 8-B pair fill)" if ext1[-1] % 2 == 0 else
                                       "K1 tile2d (cp.async 4-B fill)"),
                                   2: "K2 sweep3d (TMA)",
                                   3: "K4 persistent iterate (cooperative)",
                                   4: "K5 gather tiles",
                                   5: "K6 shared-memory-resident iterate (cooperative)"}[variant_id],
                       "launch": (f"cuda graph replay ({launches_per_step} launches per graph)" if graph is not None
                                  else "stream launches")},
            "hbm_gbs_per_gpu_whole_step": value * bpp_launch / tb / world,
            "roofline": {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                         "frac": achieved / peak, "traffic": ncu_traffic(args.workload, kernel_name),
                         "kernel": kernel_name,
                         "time_steps_per_launch": tb,
                         "single_step_roofline_gpts": peak / bpp,
                         "peak_source": peak_src,
                         "alg_bytes_per_launch": alg_bytes, "avg_launch_us": avg_launch_s * 1e6,
                         "frac_of_8TBs": achieved / 8000.0},
            "cpu_baseline": cpu,
            "halo": halo,
            "hot": hot,
            "single_step": single_step,
            "e2e": e2e,
            "gpu_launches": int(args.steps * launches_per_step),
            "clocks": clocks,
        }
        print(json.dumps(line), flush=True)
    if use_pg:
        dist.barrier()
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
