"""Fused pass-2 + join diagnostics: results of every knob combination vs the unfused path on
one config, repeated; prints mismatches and per-call times.

    python tools/fz_diag.py c1 [reps]
"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

cfg = sys.argv[1]
reps = int(sys.argv[2]) if len(sys.argv) > 2 else 5
w = W.CONFIGS[cfg]
cols = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, w.key_bytes, w.key_bytes)
ctx.set_option(hj.OPT_FUSE, 0)
ref = ctx.join(*cols, radix_bits=w.radix_bits)
ref = (ref.matches, ref.checksum)
print(cfg, "ref", ref, flush=True)
for window, slots in [(0, 1), (32, 1), (8, 1), (0, 2), (32, 2)]:
    ctx.set_option(hj.OPT_FUSE, 1)
    ctx.set_option(hj.OPT_FUSE_WINDOW_MB, window)
    ctx.set_option(hj.OPT_FUSE_PASS_SLOTS, slots)
    bad, ms = 0, []
    for _ in range(reps):
        try:
            r = ctx.join(*cols, radix_bits=w.radix_bits)
        except Exception as e:  # watchdog
            print("  error", e, flush=True)
            bad += 1
            continue
        ms.append(r.ms_kernel[3])
        bad += (r.matches, r.checksum) != ref
    print(f"  window={window} slots={slots}: {bad}/{reps} bad, fused kernel ms "
          f"{min(ms) if ms else 0:.3f}..{max(ms) if ms else 0:.3f}", flush=True)
