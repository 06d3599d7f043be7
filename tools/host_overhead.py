"""Host overhead per hj_join call: wall-clock per call vs the call's own CUDA-event time, with and
without per-phase timing events, plus a cProfile of the Python side.

    python tools/host_overhead.py [config ...]
"""
import cProfile
import os
import pstats
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402

for name in sys.argv[1:] or ["c1", "c3"]:
    w = W.CONFIGS[name]
    cols = W.torch_generate(w, device="cuda")
    for timing in (1, 0):
        ctx = hj.Context(0, w.key_bytes, w.key_bytes)
        ctx.set_option(hj.OPT_TIMING, timing)
        for _ in range(5):
            r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
        torch.cuda.synchronize()
        n = 30
        ev = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        ev[0].record()
        t0 = time.perf_counter()
        tot = 0.0
        for _ in range(n):
            r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
            tot += r.ms_total
        dt = (time.perf_counter() - t0) / n
        ev[1].record()
        torch.cuda.synchronize()
        print(f"{name} timing={timing}: wall {dt * 1e3:.3f} ms/call, stream events {ev[0].elapsed_time(ev[1]) / n:.3f} "
              f"ms/call, in-call events {tot / n:.3f} ms", flush=True)
        if timing == 1:
            pr = cProfile.Profile()
            pr.enable()
            for _ in range(n):
                ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
            pr.disable()
            st = pstats.Stats(pr)
            st.sort_stats("tottime").print_stats(8)
        ctx.close()
