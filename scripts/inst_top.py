"""Top SASS instructions by instructions executed from an ncu report (source page)."""
import csv
import subprocess
import sys

rep = sys.argv[1]
n = int(sys.argv[2]) if len(sys.argv) > 2 else 30
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
print([c for c in h][:40])
cand = [i for i, c in enumerate(h) if c.startswith("Instructions Executed") or c == "Warp Instructions Executed"]
if not cand:
    sys.exit("no instruction column")
ie = cand[0]
data = rows[2:]
def val(r):
    try:
        return float(r[ie].replace(",", ""))
    except (ValueError, IndexError):
        return 0.0
tot = sum(val(r) for r in data)
print("column", h[ie], "total", tot)
for j in sorted(range(len(data)), key=lambda j: -val(data[j]))[:n]:
    r = data[j]
    print(f"{j:5d} {val(r) / tot * 100:5.2f}%  {r[1].strip()[:70]}")
