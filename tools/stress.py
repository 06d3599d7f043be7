"""Stress: run one config's join many times and compare every result with the generator's closed
form (matches == |S|, checksum == sum_j sig(rho(j), j), computed on the host with numpy).

    python tools/stress.py c4_z0.5 --reps 30 [--pre c3] [--fresh-ctx]
"""
import argparse
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

GOLDEN = 0x9E3779B97F4A7C15


def closed_form(w):
    cdf = W.zipf_cdf(w.nR, w.z) if w.dist == "zipf" else None
    j = np.arange(w.nS, dtype=np.uint64)
    rho = W.np_rho_for(w, j, cdf)
    with np.errstate(over="ignore"):
        sig = W.np_fmix64(rho ^ (j * np.uint64(GOLDEN)))
    return w.nS, int(sig.sum(dtype=np.uint64))


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("cfg")
    ap.add_argument("--reps", type=int, default=20)
    ap.add_argument("--pre", default=None)
    ap.add_argument("--fresh-ctx", action="store_true")
    a = ap.parse_args()
    w = W.CONFIGS[a.cfg]
    t0 = time.time()
    exp = closed_form(w)
    print(f"closed form {exp} in {time.time() - t0:.1f}s", flush=True)
    ctx = hj.Context(0, 4, 4)
    if a.pre:
        wp = W.CONFIGS[a.pre]
        cols = W.torch_generate(wp, device="cuda")
        r = ctx.join(*cols, radix_bits=wp.radix_bits, out_mode=wp.out_mode)
        print("pre", a.pre, r.matches, flush=True)
        del cols, r
    cols = W.torch_generate(w, device="cuda")
    bad = 0
    for i in range(a.reps):
        if a.fresh_ctx:
            ctx = hj.Context(0, 4, 4)
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=0)
        ok = (r.matches, r.checksum) == exp
        bad += not ok
        if not ok:
            print(f"rep {i}: MISMATCH matches {r.matches} (exp {exp[0]}) checksum {r.checksum:#x} (exp {exp[1]:#x}) "
                  f"items {r.n_items}", flush=True)
    print(f"{a.cfg}: {bad} / {a.reps} mismatches", flush=True)


if __name__ == "__main__":
    main()
