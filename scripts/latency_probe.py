"""Floors for small L2-resident / cold sweeps on B200 (no stencil work):
per-launch time of a graph of 100 dependent tiny kernels, of 100 copies of an
8 MB grid (L2-resident), and one cold 24 MB-traffic copy after an L2 flush
that leaves DIRTY lines (fill_) vs CLEAN lines (fill_ then a read), plus the
same for one Hotspot3D (8,512,512) sweep."""
import json
import sys

import torch

sys.path.insert(0, ".")


def graph_time(fn, reps=100, rounds=5):
    g = torch.cuda.CUDAGraph()
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        fn()
    torch.cuda.current_stream().wait_stream(s)
    with torch.cuda.graph(g):
        for _ in range(reps):
            fn()
    best = 1e9
    for _ in range(rounds):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        g.replay()
        e1.record()
        torch.cuda.synchronize()
        best = min(best, e0.elapsed_time(e1) * 1e3 / reps)
    return best


def cold_time(fn, flush_mode, reps=20):
    L2 = 126_000_000
    fb = torch.empty(int(2 * L2) // 4, dtype=torch.int32, device="cuda")
    rb = torch.ones(int(2 * L2) // 4, dtype=torch.int32, device="cuda")
    ts = []
    for k in range(reps + 3):
        fb.fill_(k)
        if flush_mode == "clean":
            rb.sum()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        fn()
        e1.record()
        torch.cuda.synchronize()
        if k >= 3:
            ts.append(e0.elapsed_time(e1) * 1e3)
    ts.sort()
    return ts[len(ts) // 2]


def main():
    import paper_conf_cgo_hagedornssgd18_b200 as lift
    import stencil_inputs as si
    res = {}
    tiny = torch.zeros(1, device="cuda")
    res["graph_tiny_kernel_us"] = graph_time(lambda: tiny.add_(1))
    a = torch.rand(8, 512, 512, device="cuda")
    b = torch.empty_like(a)
    res["graph_copy_8MB_us"] = graph_time(lambda: b.copy_(a))
    a3 = torch.rand(3, 8, 512, 512, device="cuda")
    b3 = torch.empty(8, 512, 512, device="cuda")
    res["graph_sum3_8MB_us"] = graph_time(lambda: torch.sum(a3[:2], 0, out=b3))
    for mode in ("dirty", "clean"):
        res[f"cold_copy_8MB_{mode}_us"] = cold_time(lambda: b.copy_(a), mode)
        res[f"cold_add_16MB_to_8MB_{mode}_us"] = cold_time(lambda: torch.add(a3[0], a3[1], out=b3), mode)
    xs, spec = si.make_workload_inputs(si.workload("hotspot3d_8x512x512"))
    plan = lift.Plan.from_spec(spec)
    T, P = (torch.from_numpy(x).cuda() for x in xs)
    out = torch.empty_like(T)
    for mode in ("dirty", "clean"):
        res[f"cold_hotspot_{mode}_us"] = cold_time(lambda: plan.apply(T, P, out=out), mode)
    res["graph_hotspot_us"] = graph_time(lambda: plan.apply(T, P, out=out))
    print(json.dumps(res, indent=1))


if __name__ == "__main__":
    main()
