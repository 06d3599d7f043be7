"""Small joins for compute-sanitizer (memcheck / racecheck / synccheck / initcheck): every kernel
of the default path, materialize and count, 4/4 and 8/8, partition exports, exchange path,
streaming host path, comparators."""
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle  # noqa: E402
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a).view(np.int32 if a.dtype.itemsize == 4 else np.int64)).cuda()


def check(ctx, w, bits=-1):
    Rk, Rp, Sk, Sp = W.np_generate(w)
    m, c = oracle.hash_join(Rk, Rp, Sk, Sp)
    r = ctx.join(dev(Rk), dev(Rp), dev(Sk), dev(Sp), radix_bits=bits)
    assert (r.matches, r.checksum) == (m, c), (w, r.matches, m)
    r = ctx.join(dev(Rk), dev(Rp), dev(Sk), dev(Sp), radix_bits=bits, out_mode=1)
    assert (r.matches, r.checksum) == (m, c)
    return Rk, Rp, Sk, Sp


which = sys.argv[1] if len(sys.argv) > 1 else "all"
ctx4 = hj.Context(0, 4, 4)  # hj_join on a torch workspace (binding default)
ctx8 = hj.Context(0, 8, 8, workspace=False)  # ctx-owned buffers
cases = [W.Workload("a", 20000, 30011, "fk", keys="sparse", seed=400),
         W.Workload("b", 1 << 14, 1 << 15, "zipf", z=1.5, seed=401),
         W.Workload("c", 5000, 7000, "zipf_both", keys="sparse", z=1.0, seed=402)]
for w in cases:
    for bits in (-1, 0, 5, 11):
        check(ctx4, w, bits)
check(ctx8, W.Workload("d", 9000, 12000, "1to1", keys="k8", seed=403).with_(nS=9000))
cw = hj.Context(0, 4, 4)
cw.set_option(hj.OPT_PASS_WS, 0)  # the lock-step partition passes (racecheck covers them; see test)
check(cw, W.Workload("h", 20000, 30011, "zipf", z=1.2, keys="sparse", seed=407))
if which == "all":
    w = W.Workload("e", 30000, 40000, "fk", keys="sparse", seed=404)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    ctx4.partition(dev(Rk), dev(Rp), 9)
    ctx4.set_option(hj.OPT_STREAM_CHUNK, 7000)
    r = ctx4.join_host(Rk, Rp, Sk, Sp, out_mode=1)
    assert r.matches == oracle.hash_join(Rk, Rp, Sk, Sp)[0]
    for algo in (1, 2):
        c = hj.Context(0, 4, 4)
        c.set_option(hj.OPT_JOIN_ALGO, algo)
        check(c, W.Workload("f", 3000, 5000, "fk", keys="sparse", seed=405))
    c = hj.Context(0, 4, 4)
    c.set_option(hj.OPT_PARTITIONER, 1)  # bucket chains
    check(c, W.Workload("g", 20000, 30011, "zipf", z=1.2, keys="sparse", seed=406))
    # exchange path with 2 virtual ranks
    send, cnt, dest = ctx4.exchange_pack(0, dev(Rk), dev(Rp), 1, 6)
    torch.cuda.synchronize()
    # direct-store exchange, one rank (the sanitizers serialize kernels, so the phase waits must
    # be satisfiable by the rank itself): every hj_xd_join kernel, a regrow, both output modes
    cx = hj.Context(0, 4, 4)
    m, c, rr, ss = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
    H = hj.xd_header_bytes(1, 6)
    for scale, mode in ((0.5, 0), (1.2, 0), (1.2, 1)):
        cap = [[H + 64 + int(scale * len(Rk)) * 8], [H + 64 + int(scale * len(Sk)) * 8]]
        wr, _, _ = cx.xd_window(0, cap[0][0], want_handle=False)
        ws, _, _ = cx.xd_window(1, cap[1][0], want_handle=False)
        wb, _, _ = cx.xd_window(2, hj.XD_BOARD_BYTES, want_handle=False)
        rc, res, tot, allv = cx.xd_join(0, 0, dev(Rk), dev(Rp), dev(Sk), dev(Sp), 6, mode, [wr], [ws], [wb], cap)
        if scale < 1:
            assert rc == hj.XD_REGROW and int(tot[1].sum()) == len(Sk)
        else:
            assert rc == 0 and (allv[0], allv[1]) == (m, c)
    cx.close()
print("sanitize cases ok", flush=True)
