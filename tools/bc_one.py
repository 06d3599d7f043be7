"""One process, a sequence of joins: python tools/bc_one.py CONFIG PARTITIONER [CONFIG PARTITIONER ...]
(a fresh Context per pair, closed before the next; prints matches per pair)."""
import sys, os
sys.path.insert(0, os.getcwd())
import torch, paper_conf_icde_sioulasckaa19_b200 as hj, workloads as W
args = sys.argv[1:]
for name, part in zip(args[0::2], args[1::2]):
    w = W.CONFIGS[name]
    cols = W.torch_generate(w, device="cuda")
    ctx = hj.Context(0, w.key_bytes, w.key_bytes)
    ctx.set_option(hj.OPT_PARTITIONER, int(part))
    for _ in range(2):
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
    torch.cuda.synchronize()
    print(name, part, r.matches, flush=True)
    if not os.environ.get("KEEP"):  # KEEP=1: contexts stay open (no device memory recycled)
        ctx.close()
        del cols
