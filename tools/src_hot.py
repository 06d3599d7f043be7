"""Per-CUDA-source-line hot spots from `ncu -i R --page source --csv --print-source cuda,sass`.
usage: python tools/src_hot.py report.ncu-rep kernel_regex [N]"""
import csv
import subprocess
import sys

rep, kern = sys.argv[1], sys.argv[2]
n = int(sys.argv[3]) if len(sys.argv) > 3 else 30
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--kernel-name", f"regex:{kern}", *(["--launch-skip", sys.argv[4]] if len(sys.argv) > 4 else []),
                      "--launch-count", "1", "--print-source", "cuda,sass"], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
fname, stats = None, []
hdr = None
for r in rows:
    if not r:
        continue
    if r[0] in ("File Path", "File Name"):
        fname = r[1].split("/")[-1]
        continue
    if r[0] == "Line No":
        hdr = r
        continue
    if hdr is None or r[0] == "" or not r[0].isdigit():
        continue
    d = dict(zip(hdr, r))
    try:
        ex = float(d.get("Instructions Executed", 0) or 0)
        st = float(d.get("Warp Stall Sampling (All Samples)", 0) or 0)
    except ValueError:
        continue
    stats.append((fname, int(r[0]), r[1].strip()[:80], ex, st))
te = sum(s[3] for s in stats) or 1
ts = sum(s[4] for s in stats) or 1
print(f"total instructions {te:.3e}")
for f, ln, src, ex, st in sorted(stats, key=lambda s: -s[4])[:n]:
    print(f"{f}:{ln:<4} stall {st / ts:6.1%}  inst {ex / te:6.1%}  {src}")
