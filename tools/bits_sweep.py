"""Time one config's join at several radix_bits (results must not change).

    python tools/bits_sweep.py c5_gpu 15 16 17
"""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

w = W.CONFIGS[sys.argv[1]]
cols = W.torch_generate(w, device="cuda")
ref = None
for bits in (int(b) for b in sys.argv[2:]):
    ctx = hj.Context(0, w.key_bytes, w.key_bytes)
    for _ in range(3):
        r = ctx.join(*cols, radix_bits=bits, out_mode=w.out_mode)
    ks, tot, n = np.zeros(5), 0.0, 10
    for _ in range(n):
        r = ctx.join(*cols, radix_bits=bits, out_mode=w.out_mode)
        ks += np.array(r.ms_kernel)
        tot += r.ms_total
    ref = ref or (r.matches, r.checksum)
    ks /= n
    print(f"{w.name} bits={bits}: total {tot / n:.3f} ms  " +
          "  ".join(f"{k} {v:.3f}" for k, v in zip(["hist", "plan", "pass1", "pass2", "join"], ks)) +
          f"  items {r.n_items}  {'ok' if (r.matches, r.checksum) == ref else 'MISMATCH'}", flush=True)
    ctx.close()
    torch.cuda.synchronize()
