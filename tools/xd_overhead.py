"""Host overhead of the device-driven multi-GPU join at one rank (hj_xd_join through
dist.DirectExchange, 1-rank NCCL group) against the single-GPU hj_join on the same workload:
wall-clock per call, stream-event time per call, and a cProfile of the Python side.

    python tools/xd_overhead.py [config]
"""
import cProfile
import os
import pstats
import sys
import time

import torch
import torch.distributed as dist

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist  # noqa: E402
import workloads as W  # noqa: E402

os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
os.environ.setdefault("MASTER_PORT", "29533")
dist.init_process_group("nccl", rank=0, world_size=1)
torch.cuda.set_device(0)
w = W.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "c3"]
cols = W.torch_generate(w, device="cuda")
ctx = hj.Context(0, w.key_bytes, w.key_bytes)
xd = hjdist.DirectExchange(ctx)
lb = hjdist._local_bits(w.nR, 1)


def timed(fn, n=20):
    for _ in range(3):
        fn()
    torch.cuda.synchronize()
    ev = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    ev[0].record()
    t0 = time.perf_counter()
    for _ in range(n):
        r = fn()
    dt = (time.perf_counter() - t0) / n
    ev[1].record()
    torch.cuda.synchronize()
    return dt * 1e3, ev[0].elapsed_time(ev[1]) / n, r


for name, fn in (("hj_join", lambda: ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)),
                 ("xd_join", lambda: xd.join(*cols, local_bits=lb, out_mode=w.out_mode))):
    wall, evt, r = timed(fn)
    loc = r if name == "hj_join" else r.local
    print(f"{w.name} {name}: wall {wall:.3f} ms/call, stream {evt:.3f} ms/call, in-call {loc.ms_total:.3f} ms, "
          f"kernels {[round(x, 3) for x in loc.ms_kernel]} launches {loc.kernels}", flush=True)
pr = cProfile.Profile()
pr.enable()
for _ in range(20):
    xd.join(*cols, local_bits=lb, out_mode=w.out_mode)
pr.disable()
pstats.Stats(pr).sort_stats("tottime").print_stats(10)
xd.close()
dist.destroy_process_group()
