"""Time the join pipeline for each value of a tuning option (results must not change).

    python tools/tune.py --config c3 --opt join_variant --values 0 1 2 3 4
"""
import argparse
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

OPTS = {"join_variant": hj.OPT_JOIN_VARIANT, "cap_r": hj.OPT_CAP_R, "chunk_s": hj.OPT_CHUNK_S,
        "blocks_per_sm": hj.OPT_BLOCKS_PER_SM, "pass_threads": hj.OPT_PASS_THREADS, "join_algo": hj.OPT_JOIN_ALGO,
        "stream_chunk": hj.OPT_STREAM_CHUNK, "partitioner": hj.OPT_PARTITIONER,
        "pass_l2pf": hj.OPT_PASS_L2PF, "pass1_bits": hj.OPT_PASS1_BITS,
        "pass_variant": hj.OPT_PASS_VARIANT, "mat_checksum": hj.OPT_MAT_CHECKSUM, "pass_ws": hj.OPT_PASS_WS,
        "pdl": hj.OPT_PDL, "timing": hj.OPT_TIMING}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--config", default="c3")
    ap.add_argument("--opt", default="join_variant")
    ap.add_argument("--values", type=int, nargs="+", default=[0])
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--bits", type=int, default=None, help="radix bits instead of the config's")
    a = ap.parse_args()
    w = W.CONFIGS[a.config]
    if a.bits is not None:
        w = w.with_(radix_bits=a.bits)
    cols = W.torch_generate(w, device="cuda")
    ref = None
    for v in a.values:  # join_variant: 0 = auto, k = shape k-1
        ctx = hj.Context(0, w.key_bytes, w.key_bytes)
        ctx.set_option(OPTS[a.opt], v)
        for _ in range(3):
            r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
        ks = np.zeros(5)
        tot = 0.0
        for _ in range(a.steps):
            r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
            ks += np.array(r.ms_kernel)
            tot += r.ms_total
        key = (r.matches, r.checksum)
        ref = ref or key
        ok = "ok" if key == ref else "MISMATCH"
        ks /= a.steps
        print(f"{a.config} {a.opt}={v}: total {tot / a.steps:.3f} ms  hist {ks[0]:.3f} plan {ks[1]:.3f} "
              f"pass1 {ks[2]:.3f} pass2 {ks[3]:.3f} join {ks[4]:.3f}  items {r.n_items}  {ok}", flush=True)
        ctx.close()


if __name__ == "__main__":
    main()
