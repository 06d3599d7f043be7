"""Turn the round's ncu captures into the committed evidence under profiles/.

    python tools/profile_summary.py ROUND LAUNCHES.csv FULL.ncu-rep CONFIG
writes profiles/<ROUND>_launches_<CONFIG>.csv (our kernels only: name, grid, block, ms, DRAM bytes),
profiles/<ROUND>_ncu_<CONFIG>.md and profiles/traffic_<CONFIG>.json (DRAM bytes per launch of
each kernel of the last complete step, read by bench.py as roofline.traffic).
"""
import csv
import json
import os
import subprocess
import sys

sys.path.insert(0, os.path.dirname(os.path.abspath(__file__)))
from ncu_summary import main as ncu_main  # noqa: E402

NAMES = {"k_hist": "hist", "k_plan": "plan", "k_pass": None, "k_join": "join"}


def short(name):
    if "k_pass" in name:
        return "pass1" if ", 1," in name or "(int)1," in name else "pass2"
    for k, v in NAMES.items():
        if k in name and v:
            return v
    return None


def main(rnd, launches, rep, cfg, outdir="profiles"):
    rows = list(csv.reader(open(launches)))
    rows = [r for r in rows if len(r) > 14 and r[0].isdigit()]
    hdr = ["ID", "Process ID", "Process Name", "Host Name", "Kernel Name", "Context", "Stream", "Block Size",
           "Grid Size", "Device", "CC", "Section Name", "Metric Name", "Metric Unit", "Metric Value"]
    per = {}
    for r in rows:
        d = dict(zip(hdr, r))
        if not short(d["Kernel Name"]):
            continue
        e = per.setdefault(d["ID"], {"kernel": short(d["Kernel Name"]), "name": d["Kernel Name"][:80],
                                     "grid": d["Grid Size"], "block": d["Block Size"]})
        v = float(d["Metric Value"].replace(",", ""))
        unit = d["Metric Unit"]
        if d["Metric Name"] == "gpu__time_duration.sum":
            e["ms"] = v / 1e6 if unit == "ns" else (v / 1e3 if unit == "us" else v)
        else:
            scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}.get(unit, 1)
            e[d["Metric Name"]] = v * scale
    out = os.path.join(outdir, f"{rnd}_launches_{cfg}.csv")
    with open(out, "w") as f:
        w = csv.writer(f)
        w.writerow(["launch_id", "kernel", "grid", "block", "ms", "dram_read_bytes", "dram_write_bytes", "name"])
        for k in sorted(per, key=int):
            e = per[k]
            w.writerow([k, e["kernel"], e["grid"], e["block"], f"{e.get('ms', 0):.4f}",
                        int(e.get("dram__bytes_read.sum", 0)), int(e.get("dram__bytes_write.sum", 0)), e["name"]])
    # traffic of the last step's launches
    last = {}
    for k in sorted(per, key=int):
        last[per[k]["kernel"]] = per[k].get("dram__bytes_read.sum", 0) + per[k].get("dram__bytes_write.sum", 0)
    json.dump({k: int(v) for k, v in last.items()}, open(os.path.join(outdir, f"traffic_{cfg}.json"), "w"),
              indent=1)
    # full-set summary
    import io
    from contextlib import redirect_stdout

    buf = io.StringIO()
    with redirect_stdout(buf):
        ncu_main(rep)
    with open(os.path.join(outdir, f"{rnd}_ncu_{cfg}.md"), "w") as f:
        f.write(f"# ncu --set full summary, {rnd}, config {cfg} (one step, cold-cache serialized replays)\n\n")
        f.write("```\n" + buf.getvalue() + "```\n")
    print(open(out).read())
    print(json.dumps(last))


if __name__ == "__main__":
    a = sys.argv[1:]
    od = "profiles"
    if "--outdir" in a:
        i = a.index("--outdir")
        od = a[i + 1]
        del a[i:i + 2]
    main(*a[:4], outdir=od)
