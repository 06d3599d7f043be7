"""Host time per call vs device time: how much of a step is the synchronous call's round trip.
    python tools/host_overhead.py [config]"""
import ctypes
import os
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

w = W.CONFIGS[sys.argv[1] if len(sys.argv) > 1 else "c1"]
cols = W.torch_generate(w, device="cuda")
torch.cuda.synchronize()
for graph in (0, 1):
    ctx = hj.Context(0, w.key_bytes, w.key_bytes)
    ctx.set_option(hj.OPT_GRAPH, graph)
    for _ in range(5):
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
    N = 50
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    t0 = time.perf_counter()
    e0.record()
    dev = 0.0
    for _ in range(N):
        r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
        dev += r.ms_total
    e1.record()
    torch.cuda.synchronize()
    wall = (time.perf_counter() - t0) / N * 1e3
    # the raw C call with marshalled arguments (no binding work)
    res = hj._Result()
    args = [ctx._h] + [ctypes.c_void_p(c.data_ptr()) for c in cols]
    t1 = time.perf_counter()
    for _ in range(N):
        hj.lib().hj_join(args[0], args[1], args[2], w.nR, args[3], args[4], w.nS, w.radix_bits, w.out_mode,
                         ctypes.byref(res))
    raw = (time.perf_counter() - t1) / N * 1e3
    print(f"{w.name} graph={graph}: device events {e0.elapsed_time(e1) / N:.3f} ms/call, in-call ms_total "
          f"{dev / N:.3f}, wall {wall:.3f} ms/call, raw C-ABI call {raw:.3f} ms/call, "
          f"kernels {[round(x, 3) for x in r.ms_kernel]}", flush=True)
    ctx.close()
