"""Per-kernel summary of an ncu --set full report: duration, DRAM bytes, occupancy, stall mix."""
import csv
import subprocess
import sys

WANT = ["gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
        "dram__throughput.avg.pct_of_peak_sustained_elapsed", "sm__warps_active.avg.pct_of_peak_sustained_active",
        "launch__registers_per_thread", "launch__grid_size", "launch__block_size", "smsp__inst_executed.sum",
        "sm__throughput.avg.pct_of_peak_sustained_elapsed",
        "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum",
        "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum",
        "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_atom.sum",
        "lts__t_sectors_op_write.sum", "lts__t_requests_op_write.sum", "lts__t_sectors_op_read.sum",
        "smsp__sass_inst_executed_op_shared_atom.sum", "l1tex__data_pipe_lsu_wavefronts_mem_shared.sum"]


def main(path, as_json=False):
    out = subprocess.run(["ncu", "-i", path, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    rows = list(csv.reader(out.splitlines()))
    hdr, units, data = rows[0], rows[1], rows[2:]
    stall = [i for i, h in enumerate(hdr) if h.startswith("smsp__average_warps_issue_stalled") and
             h.endswith("_per_issue_active.ratio")]
    res = []
    for r in data:
        d = {"kernel": r[hdr.index("Kernel Name")]}
        for w in WANT:
            if w in hdr:
                i = hdr.index(w)
                d[w] = f"{r[i]} {units[i]}".strip()
        def val(name, scale):
            if name not in hdr:
                return None
            i = hdr.index(name)
            u = units[i].lower()
            f = {"byte": 1, "kbyte": 1e3, "mbyte": 1e6, "gbyte": 1e9, "nsecond": 1e-9, "usecond": 1e-6,
                 "msecond": 1e-3, "second": 1, "ns": 1e-9, "us": 1e-6, "ms": 1e-3, "s": 1}.get(u, scale)
            return float(r[i].replace(",", "") or 0) * f
        rd, wr = val("dram__bytes_read.sum", 1), val("dram__bytes_write.sum", 1)
        t = val("gpu__time_duration.sum", 1e-9)
        if rd is not None and wr is not None and t:
            d["achieved_dram_GBps"] = f"{(rd + wr) / t / 1e9:.0f} GB/s (read + write / duration; cold-cache replay)"
        ws, wq = val("lts__t_sectors_op_write.sum", 1), val("lts__t_requests_op_write.sum", 1)
        if ws and wq:
            d["l2_write_sectors_per_request"] = f"{ws / wq:.2f} (4 = full 128-byte lines per request)"
        st = sorted(((float(r[i] or 0), hdr[i].replace("smsp__average_warps_issue_stalled_", "")
                      .replace("_per_issue_active.ratio", "")) for i in stall), reverse=True)[:6]
        d["top_stalls"] = ", ".join(f"{n}={v:.2f}" for v, n in st)
        res.append(d)
    for d in res:
        print("==", d["kernel"])
        for k, v in d.items():
            if k != "kernel":
                print(f"   {k}: {v}")
    return res


if __name__ == "__main__":
    main(sys.argv[1])
