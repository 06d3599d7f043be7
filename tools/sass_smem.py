"""Shared-memory wavefronts per SASS instruction of one kernel in an ncu report (--set full).
usage: python tools/sass_smem.py report.ncu-rep kernel_regex [N]
Prints the instructions with the most L1 shared wavefronts: executed count, wavefronts, ideal,
stall samples -- where a pass's shared-memory pipe time goes."""
import csv
import subprocess
import sys

rep, kern = sys.argv[1], sys.argv[2]
n = int(sys.argv[3]) if len(sys.argv) > 3 else 25
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "--kernel-name", f"regex:{kern}",
                      "--launch-count", "1", "--print-source", "sass"], capture_output=True, text=True).stdout
rows = list(csv.reader(out.splitlines()))
hdr = rows[1]
ix = {h: i for i, h in enumerate(hdr)}
recs = []
for r in rows[2:]:
    if len(r) < len(hdr) or r[0] == "Address" or not r[0].startswith("0x"):
        continue
    f = lambda k: float(r[ix[k]] or 0) if r[ix[k]] not in ("-", "") else 0.0
    recs.append((r[ix["Address"]][-5:], r[ix["Source"]].strip()[:60], f("Instructions Executed"),
                 f("L1 Wavefronts Shared"), f("L1 Wavefronts Shared Ideal"), f("Warp Stall Sampling (All Samples)")))
tw = sum(x[3] for x in recs) or 1
ts = sum(x[5] for x in recs) or 1
print(f"total shared wavefronts {tw:.4e}, stall samples {ts:.0f}")
for a, s, ex, wf, wi, st in sorted(recs, key=lambda x: -x[3])[:n]:
    print(f"{a} {s:60s} exec {ex:10.0f} wf {wf:11.0f} ({wf / tw:5.1%}) ideal {wi:11.0f} wf/inst {wf / max(ex, 1):5.2f} stall {st / ts:5.1%}")

# by opcode (first token after the predicate), addresses de-duplicated
seen, agg = set(), {}
for a, s, ex, wf, wi, st in recs:
    if a in seen:
        continue
    seen.add(a)
    toks = [t for t in s.split() if not t.startswith("@")]
    op = toks[0] if toks else "?"
    e = agg.setdefault(op, [0, 0, 0, 0])
    e[0] += ex; e[1] += wf; e[2] += wi; e[3] += st
tw2 = sum(e[1] for e in agg.values()) or 1
print("\nby opcode:")
for op, (ex, wf, wi, st) in sorted(agg.items(), key=lambda kv: -kv[1][1])[:15]:
    if wf:
        print(f"  {op:14s} exec {ex:11.0f} wf {wf:11.0f} ({wf / tw2:5.1%}) ideal {wi:11.0f} wf/inst {wf / max(ex, 1):5.2f}")
