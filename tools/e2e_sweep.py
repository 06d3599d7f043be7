"""e2e (hj_join_host from pinned host memory) vs the streaming chunk size."""
import os
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

w = W.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "c3"]
cols = W.torch_generate(w, device="cuda")
host = []
for t in cols:
    h = torch.empty(t.shape, dtype=t.dtype, pin_memory=True)
    h.copy_(t)
    host.append(h.numpy())
del cols
for chunk in [0, w.nS // 4, w.nS // 16, w.nS // 32, w.nS // 64, w.nS]:
    ctx = hj.Context(0, w.key_bytes, w.key_bytes)
    ctx.set_option(hj.OPT_STREAM_CHUNK, chunk)
    r = ctx.join_host(*host, radix_bits=w.radix_bits, out_mode=w.out_mode, copy=False)
    t0 = time.perf_counter()
    for _ in range(3):
        r = ctx.join_host(*host, radix_bits=w.radix_bits, out_mode=w.out_mode, copy=False)
    dt = (time.perf_counter() - t0) / 3
    print(f"chunk {chunk}: {dt * 1e3:.1f} ms  {w.n / dt / 1e9:.2f} G tuples/s  (event {r.ms_total:.1f} ms)", flush=True)
    ctx.close()
