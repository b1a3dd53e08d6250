"""Top SASS instructions by warp-stall samples from an ncu report (source page)."""
import csv
import subprocess
import sys

rep = sys.argv[1]
n = int(sys.argv[2]) if len(sys.argv) > 2 else 25
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
data = rows[2:]
si = h.index("Warp Stall Sampling (All Samples)")
cols = [i for i, k in enumerate(h) if k.startswith("stall_") and "Not Issued" not in k]
tot = sum(int(r[si]) for r in data if r[si].isdigit())
print("total samples", tot)
agg = {}
for r in data:
    for i in cols:
        if r[i].isdigit():
            agg[h[i]] = agg.get(h[i], 0) + int(r[i])
print("by reason:", ", ".join(f"{k[6:]} {100*v/tot:.1f}%" for k, v in sorted(agg.items(), key=lambda x: -x[1])[:8]))
top = sorted(range(len(data)), key=lambda j: -int(data[j][si]) if data[j][si].isdigit() else 0)[:n]
for j in sorted(top):
    r = data[j]
    why = sorted(((int(r[i]), h[i][6:]) for i in cols if r[i].isdigit() and int(r[i]) > 0), reverse=True)[:2]
    print(f"{j:5d} {int(r[si]):6d} {r[1].strip()[:60]:60s} {why}")
