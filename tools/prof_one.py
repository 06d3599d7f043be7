"""One warm-up join and one profiled join of a bench config (for ncu captures):
    ncu -k regex:k_pass --launch-skip 2 --launch-count 2 python tools/prof_one.py c3 [opt=value ...]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

w = W.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "c3"]
cols = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, w.key_bytes, w.key_bytes)
for kv in sys.argv[2:]:
    k, v = kv.split("=")
    ctx.set_option(getattr(hj, "OPT_" + k.upper()), int(v))
for _ in range(2):
    r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
torch.cuda.synchronize()
print(w.name, r.matches, r.checksum, [round(x, 3) for x in r.ms_kernel])
