import sys, os
sys.path.insert(0, os.getcwd())
import torch, paper_conf_icde_sioulasckaa19_b200 as hj, workloads as W
w = W.CONFIGS[sys.argv[1]]
cols = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, w.key_bytes, w.key_bytes)
ctx.set_option(hj.OPT_PARTITIONER, int(sys.argv[2]))
for _ in range(2):
    r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
torch.cuda.synchronize()
print(r.matches)
