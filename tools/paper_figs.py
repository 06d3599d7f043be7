"""Re-measure the paper's GPU-resident comparisons on B200 (SURVEY NEXT-4 / experiments E5, E8).

  Fig. 5: nested loops (ballot, Listing 1) vs hash join for the co-partition
         join, 2M unique uniform keys per table, partition sizes 256..2048 -> radix bits 13..10.
  Fig. 8: partitioned vs non-partitioned GPU hash join, equal sizes 1M..128M,
         1:1 unique keys, aggregation (count + checksum).

  Fig. 17: Zipf skew on GPU-resident data, 32M tuples per
         table, z = 0 .. 1, skew on the probe side, the build side, or identical on both;
         aggregation and materialization.
  Fig. 19: uniform duplicates (every key replicated k times on both sides).

Prints a markdown table; every row is checked against the closed form (matches == |S|, |R|,
|R| * k) or, for identical skew, against sum_k c_R(k) c_S(k) computed with torch.unique.
    python tools/paper_figs.py [--fig 5|8|17|19|all]
"""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

ALGO = {0: "radix + smem hash", 1: "radix + ballot NLJ", 2: "non-partitioned"}


def run(w, algo, bits, steps=5, out_mode=0, cols=None, expect=None):
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_JOIN_ALGO, algo)
    cols = cols if cols is not None else W.torch_generate(w, device="cuda")
    for _ in range(2):
        r = ctx.join(*cols, radix_bits=bits, out_mode=out_mode)
    ms = 0.0
    for _ in range(steps):
        r = ctx.join(*cols, radix_bits=bits, out_mode=out_mode)
        ms += r.ms_total
    ms /= steps
    assert r.matches == (w.nS if expect is None else expect), (r.matches, expect)
    ctx.close()
    return ms, r


def bag_matches(Rk, Sk):
    """sum over keys of c_R(k) * c_S(k) (torch library primitives; independent of the kernels)."""
    import torch

    ur, cr = torch.unique(Rk, return_counts=True)
    us, cs = torch.unique(Sk, return_counts=True)
    pos = torch.searchsorted(us, ur).clamp(max=len(us) - 1)
    hit = us[pos] == ur
    return int((cr[hit] * cs[pos[hit]]).sum())


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

    if a.fig in ("17", "all"):
        n = 32 << 20
        print("\n### Fig. 17 analogue: Zipf skew, GPU-resident, 32M x 32M (B200)\n")
        print("| skew | z | output | matches | ms | G tuples/s |")
        print("|---|---|---|---|---|---|")
        arms = [("probe", "zipf"), ("build", "zipf_build"), ("identical", "zipf_both")]
        for arm, dist in arms:
            for z in (0.0, 0.25, 0.5, 0.75, 1.0):
                if arm == "identical" and z >= 1.0:  # ~5.8e12 matches: all-against-all for minutes
                    print(f"| {arm} | {z} | aggregation | ~5.8e12 (collapse) | not run | |", flush=True)
                    continue
                zz = z if z > 0 else 1e-9  # z = 0: uniform ranks through the same generator
                w = W.Workload("f17", n, n, dist, keys="sparse", z=zz, seed=320)
                cols = W.torch_generate(w, device="cuda")
                exp = W.expected_matches_closed_form(w)
                if exp is None:
                    exp = bag_matches(cols[0], cols[2])
                heavy = exp > 8 * n
                for out_mode, name in ((0, "aggregation"), (1, "materialization")):
                    if out_mode and exp > 4 * n:  # the pairs would not fit next to the inputs
                        print(f"| {arm} | {z} | {name} | {exp} | not run (output > HBM budget) | |", flush=True)
                        continue
                    ms, r = run(w, 0, -1, steps=1 if heavy else 5, out_mode=out_mode, cols=cols, expect=exp)
                    print(f"| {arm} | {z} | {name} | {r.matches} | {ms:.3f} | {w.n / ms / 1e6:.1f} |", flush=True)
                del cols
    if a.fig in ("19", "all"):
        n = 32 << 20
        print("\n### Fig. 19 analogue: uniform replicas, GPU-resident, 32M x 32M (B200)\n")
        print("| replicas per key | output | matches | ms | G tuples/s |")
        print("|---|---|---|---|---|")
        for rep in (1, 2, 3, 4):
            w = W.Workload("f19", n, n, "replicas", keys="sparse", rep=rep, seed=321)
            cols = W.torch_generate(w, device="cuda")
            exp = W.expected_matches_closed_form(w)
            if exp is None:
                exp = bag_matches(cols[0], cols[2])
            for out_mode, name in ((0, "aggregation"), (1, "materialization")):
                ms, r = run(w, 0, -1, out_mode=out_mode, cols=cols, expect=exp)
                print(f"| {rep} | {name} | {r.matches} | {ms:.3f} | {w.n / ms / 1e6:.1f} |", flush=True)
            del cols


if __name__ == "__main__":
    main()
