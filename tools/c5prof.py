import sys; sys.path.insert(0,".")
import torch, workloads as W, paper_conf_icde_sioulasckaa19_b200 as hj
w = W.CONFIGS["c5_gpu"]
cols = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, 8, 8); ctx.set_option(hj.OPT_JOIN_VARIANT, 6)
for _ in range(2): r = ctx.join(*cols, radix_bits=16)
print(r.ms_kernel)
