"""Re-measure the paper's GPU-resident comparisons on B200 (SURVEY NEXT-4 / experiments E5, E8).

  Fig. 5: nested loops (ballot, Listing 1) vs hash join for the co-partition
         join, 2M unique uniform keys per table, partition sizes 256..2048 -> radix bits 13..10.
  Fig. 8: partitioned vs non-partitioned GPU hash join, equal sizes 1M..128M,
         1:1 unique keys, aggregation (count + checksum).

Prints a markdown table; every row is checked against the closed form (matches == |S|).
    python tools/paper_figs.py [--fig 5|8|all]
"""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

ALGO = {0: "radix + smem hash", 1: "radix + ballot NLJ", 2: "non-partitioned"}


def run(w, algo, bits, steps=5):
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_JOIN_ALGO, algo)
    cols = W.torch_generate(w, device="cuda")
    for _ in range(2):
        r = ctx.join(*cols, radix_bits=bits)
    ms = 0.0
    for _ in range(steps):
        r = ctx.join(*cols, radix_bits=bits)
        ms += r.ms_total
    ms /= steps
    assert r.matches == w.nS
    ctx.close()
    return ms, r


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--fig", default="all")
    a = ap.parse_args()
    if a.fig in ("5", "all"):
        print("### Fig. 5 analogue: co-partition join, 2M x 2M unique keys (B200)\n")
        print("| partition size | radix bits | algorithm | total ms | join ms | G tuples/s total | G tuples/s join |")
        print("|---|---|---|---|---|---|---|")
        w = W.Workload("f5", 1 << 21, 1 << 21, "1to1", seed=300)
        for bits in (13, 12, 11, 10):
            for algo in (1, 0):
                ms, r = run(w, algo, bits)
                print(f"| {w.nR >> bits} | {bits} | {ALGO[algo]} | {ms:.3f} | {r.ms_kernel[4]:.3f} | "
                      f"{w.n / ms / 1e6:.1f} | {w.n / r.ms_kernel[4] / 1e6:.1f} |", flush=True)
    if a.fig in ("8", "all"):
        print("\n### Fig. 8 analogue: partitioned vs non-partitioned GPU join, 1:1 unique keys (B200)\n")
        print("| tuples per relation | algorithm | ms | G tuples/s |")
        print("|---|---|---|---|")
        for lg in (20, 22, 23, 24, 25, 27):
            w = W.Workload("f8", 1 << lg, 1 << lg, "1to1", seed=301)  # the paper's dense unique keys
            for algo in ((0, 2) if lg <= 25 else (0,)):  # non-partitioned at 2^27: minutes per call
                ms, r = run(w, algo, -1)
                print(f"| 2^{lg} | {ALGO[algo]} | {ms:.3f} | {w.n / ms / 1e6:.1f} |", flush=True)


if __name__ == "__main__":
    main()
