"""Executed-instruction histogram by SASS opcode from an ncu report (source page)."""
import csv
import subprocess
import sys
from collections import Counter

rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
ie = h.index("Instructions Executed")
src = h.index("Source")
c = Counter()
tot = 0
for r in rows[2:]:
    try:
        n = int(r[ie])
    except (ValueError, IndexError):
        continue
    t = r[src].strip().split()
    if not t:
        continue
    op = t[1] if t[0].startswith("@") and len(t) > 1 else t[0]
    op = op.split(".")[0]
    c[op] += n
    tot += n
print(f"total warp-instructions {tot}")
for op, n in c.most_common(40):
    print(f"{op:12s} {n:12d} {100 * n / tot:5.1f}%")
