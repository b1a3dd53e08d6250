"""Per-config DRAM bytes per output point vs the compulsory minimum (ncu).

Runs under gpurun: for each workload, profiles 3 launches of the dominant
kernel after warm-up with dram__bytes_{read,write}.sum and
gpu__time_duration.sum (--clock-control none, cache control all), and writes
gpurun_out/ncu_bytes.json."""
import csv
import json
import subprocess
import sys

import numpy as np

sys.path.insert(0, ".")
import stencil_inputs as si  # noqa: E402

BPP = {0: 8, 1: 12, 2: 8, 3: 12, 4: 12, 5: 12, 6: 8, 7: 8}
WORKLOADS = sys.argv[1:] or ["j3d7_512_clamp", "gauss5_8192_mirror", "acoustic7_1024", "acoustic13_1024",
                             "srad1_4096", "srad2_4096", "t1_hotspot2d_8192", "t1_gradient_8192",
                             "t1_jacobi3d13_512", "t1_poisson19_512", "t1_stencil2d_4098", "srad_iter_4096",
                             "t1_jacobi2d5_8192", "t1_jacobi2d9_8192", "t1_heat7_512", "hotspot3d_8x512x512",
                             "hotspot3d_8x512x512_x100", "j2d5_256_clamp"]
out = {}
for wl in WORKLOADS:
    w = si.workload(wl)
    npts = int(np.prod(w.spec.out_extents()))
    kern = "regex:k1_srad|k1_tile|k2_sweep|k2c_column|k2t|k2r|k0_generic|k3_wsweep|k4_iterate|k6_resident|k5_gather"
    skip = "6" if w.steps > 1 else "2"     # single sweeps: 3 warm-up + 1 timed launch
    cmd = ["ncu", "--metrics", "dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum",
           "--clock-control", "none", "-k", kern, "-s", skip, "-c", "2", "--csv",
           sys.executable, "bench.py", "--workload", wl, "--steps", "1", "--warmup", "3", "--no-e2e", "--no-cpu",
           "--no-graph"]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=900)
    lines = r.stdout.splitlines()
    start = [i for i, l in enumerate(lines) if l.startswith('"ID"')]
    if not start:
        out[wl] = {"error": r.stderr[-300:]}
        continue
    rows = list(csv.reader(lines[start[0]:]))
    h = rows[0]
    vals = {}
    kname = None
    for row in rows[1:]:
        if len(row) < len(h):
            continue
        m = row[h.index("Metric Name")]
        v = float(row[h.index("Metric Value")].replace(",", ""))
        unit = row[h.index("Metric Unit")]
        scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "ns": 1, "us": 1e3, "ms": 1e6}.get(unit, 1)
        vals.setdefault(m, []).append(v * scale)
        kname = row[h.index("Kernel Name")].split("(")[0]
    rd = float(np.median(vals["dram__bytes_read.sum"]))
    wr = float(np.median(vals["dram__bytes_write.sum"]))
    t = float(np.median(vals["gpu__time_duration.sum"]))
    out[wl] = {"kernel": kname, "points": npts, "dram_read_bytes": rd, "dram_write_bytes": wr,
               "dram_bytes_per_point": (rd + wr) / npts, "compulsory_bytes_per_point": BPP[w.spec.op],
               "duration_ns_cold": t, "dram_gbs_cold": (rd + wr) / t}
    print(wl, json.dumps(out[wl]), flush=True)
json.dump(out, open("gpurun_out/ncu_bytes.json", "w"), indent=1)
# the per-launch traffic bench.py reports as roofline.traffic
traffic = {"_source": "ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum --clock-control none: median of 2 "
                      "launches of the dominant kernel after warm-up (scripts/ncu_bytes.py); "
                      "dram_bytes_per_launch = read + write"}
for wl, d in out.items():
    if "error" not in d:
        traffic[wl] = {"kernel": d["kernel"], "dram_bytes_per_launch": int(d["dram_read_bytes"] + d["dram_write_bytes"]),
                       "dram_bytes_per_point": round(d["dram_bytes_per_point"], 3),
                       "compulsory_bytes_per_point": d["compulsory_bytes_per_point"]}
json.dump(traffic, open("gpurun_out/ncu_traffic.json", "w"), indent=1)
