"""Device time per queued call (K hj_join_async + one hj_sync between two stream events) for
option settings, e.g. programmatic dependent launch and per-kernel timing events:
    python tools/pdl_check.py c3 pdl=0,timing=1 pdl=1,timing=1 pdl=0,timing=0 pdl=1,timing=0"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

w = W.CONFIGS[sys.argv[1]]
cols = W.torch_generate(w, device="cuda")
torch.cuda.synchronize()
K = 30
for rep in range(2):
    for setting in sys.argv[2:]:
        ctx = hj.Context(0, w.key_bytes, w.key_bytes)
        for kv in setting.split(","):
            k, v = kv.split("=")
            ctx.set_option(getattr(hj, "OPT_" + k.upper()), int(v))
        for _ in range(3):
            ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        torch.cuda.synchronize()
        e0.record()
        for _ in range(K):
            ctx.join_async(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
        outs = ctx.sync()
        e1.record()
        torch.cuda.synchronize()
        r = outs[-1]
        ks = [round(x, 3) for x in r.ms_kernel] if r.ms_kernel else []
        print(f"{w.name} {setting}: {e0.elapsed_time(e1) / K:.4f} ms/call  matches {r.matches} "
              f"checksum {r.checksum:#x}  kernels {ks}", flush=True)
        ctx.close()
