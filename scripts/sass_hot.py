"""Per-opcode histogram of the hottest SASS block of an ncu report (source page)."""
import csv
import subprocess
import sys
from collections import Counter

rep = sys.argv[1]
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source", "sass"],
                     capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
h = rows[1]
data = rows[2:]
ie = h.index("Instructions Executed")
src = h.index("Source")
cnt = [(int(r[ie]) if r[ie].isdigit() else 0, r[src].strip()) for r in data]
tot = sum(c for c, _ in cnt)
by = Counter()
for c, _ in cnt:
    by[c] += c
top = by.most_common(6)
print("total warp instructions", tot)
for c, w in top:
    print(f"  count {c:>12d}: {w / tot * 100:5.1f}% of instructions, {w // c} static instrs")
c0 = int(sys.argv[2]) if len(sys.argv) > 2 else top[0][0]
ops = Counter()
for c, s in cnt:
    if c == c0:
        t = s.split()
        op = t[1] if t[0].startswith("@") else t[0]
        ops[op.split(".")[0]] += 1
print(f"block with count {c0}: {sum(ops.values())} instrs")
print(" ", ", ".join(f"{k} {v}" for k, v in ops.most_common()))
if len(sys.argv) > 3:
    for c, s in cnt:
        if c == c0:
            print("   ", s[:100])
