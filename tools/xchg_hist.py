"""Exchange sender at c5's bits on one GPU: hj_exchange_pack (histogram over the (rank, d1) pieces,
planner, pass 1 into the send buffer) of 2^29 8-byte keys with gpu_bits = 3, local_bits = 16,
and the receiver's own histogram (hj_join_received on what rank 0 would receive). Prints the
CUDA-event time per call; run under `ncu --metrics gpu__time_duration.sum` for the per-kernel split.
    python tools/xchg_hist.py [log2 n]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

lg = int(sys.argv[1]) if len(sys.argv) > 1 else 29
w = W.Workload("x", 1 << lg, 1 << lg, "1to1", keys="k8", seed=109)
Rk, Rp, _, _ = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, 8, 8)
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
for it in range(4):
    e0.record()
    send, cnt, dest = ctx.exchange_pack(0, Rk, Rp, 3, 16)
    e1.record()
    torch.cuda.synchronize()
    print(f"exchange_pack 2^{lg} 8-byte keys, G=8, local_bits=16: {e0.elapsed_time(e1):.3f} ms "
          f"(rows {tuple(cnt.shape)}, to rank 0: {int(dest[0])})", flush=True)
# what rank 0 receives from this one sender: segment 0 of the send buffer
n0 = int(dest[0])
words = send[: n0 * 2].clone()
rows = torch.zeros_like(cnt)  # 8 sources; only this one sent anything
rows[0] = cnt[0]
for it in range(3):
    e0.record()
    r = ctx.join_received(words, n0, rows, words, n0, rows, 8, 16)
    e1.record()
    torch.cuda.synchronize()
    print(f"join_received of rank 0's {n0} tuples (self-join, receiver histogram over 2^16 bins): "
          f"{e0.elapsed_time(e1):.3f} ms, matches {r.matches}, kernels ms {[round(x, 3) for x in r.ms_kernel]}", flush=True)
