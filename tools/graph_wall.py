import os, sys, time, torch
sys.path.insert(0, os.getcwd())
import paper_conf_icde_sioulasckaa19_b200 as hj, workloads as W
w = W.CONFIGS["c3"]
cols = W.torch_generate(w, device="cuda")
for g in (0, 1, 0, 1):
    ctx = hj.Context(0, 4, 4)
    ctx.set_option(hj.OPT_GRAPH, g)
    for _ in range(3): ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(); t0 = time.perf_counter()
    for _ in range(30): r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
    dt = (time.perf_counter() - t0) / 30; e1.record(); torch.cuda.synchronize()
    print(f"graph={g}: wall {dt*1e3:.3f} ms/call, stream {e0.elapsed_time(e1)/30:.3f}, in-call {r.ms_total:.3f} kernels {r.ms_kernel}", flush=True)
    ctx.close()
