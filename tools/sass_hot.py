"""Summarise an `ncu --page source --print-source sass --csv` dump: hottest instructions by
warp-stall samples, and executed-instruction totals by opcode."""
import csv
import sys
from collections import Counter

rows = list(csv.reader(open(sys.argv[1])))
hdr = rows[1]
def num(x):
    try:
        float(x or 0)
        return True
    except ValueError:
        return False


data = [r for r in rows[2:] if len(r) == len(hdr) and num(r[hdr.index("Instructions Executed")])]
iS, iE, iA = hdr.index("Source"), hdr.index("Instructions Executed"), hdr.index("Address")
iW = hdr.index("Warp Stall Sampling (All Samples)")
tot_s = sum(float(r[iW] or 0) for r in data)
tot_e = sum(float(r[iE] or 0) for r in data)
print(f"instructions executed {tot_e:.3e}, stall samples {tot_s:.0f}")
ops = Counter()
for r in data:
    op = r[iS].split()[0] if r[iS].split() else "?"
    if op.startswith("@"):
        op = r[iS].split()[1]
    ops[op.split(".")[0]] += float(r[iE] or 0)
print("by opcode:", ", ".join(f"{k}={v / tot_e:.1%}" for k, v in ops.most_common(18)))
n = int(sys.argv[2]) if len(sys.argv) > 2 else 25
top = sorted(range(len(data)), key=lambda i: -float(data[i][iW] or 0))[:n]
for i in sorted(top):
    r = data[i]
    print(f"{r[iA]:>6} {float(r[iW] or 0) / tot_s:6.1%}  exec={float(r[iE] or 0):.2e}  {r[iS][:90]}")
