"""Wall-clock and event timing of small joins (launch-bound regime)."""
import os
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

for name in ["c1"] + sys.argv[1:]:
    w = W.CONFIGS[name] if name in W.CONFIGS else W.Workload(name, 1 << int(name), 1 << int(name), "fk", seed=9)
    cols = W.torch_generate(w, device="cuda")
    ctx = hj.Context(0, 4, 4)
    for _ in range(5):
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    n = 50
    ev = 0.0
    for _ in range(n):
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
        ev += r.ms_total
    dt = (time.perf_counter() - t0) / n
    print(f"{name}: wall {dt * 1e3:.3f} ms/call  events {ev / n:.3f} ms  kernels {[round(x, 4) for x in r.ms_kernel]}  "
          f"{w.n / dt / 1e9:.1f} G tuples/s", flush=True)
