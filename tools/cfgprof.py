"""Run one config's join twice (for ncu captures of its kernels)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

w = W.CONFIGS[sys.argv[1]]
cols = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, w.key_bytes, w.key_bytes)
for _ in range(2):
    r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
print(r.ms_kernel)
