import sys, numpy as np, torch
sys.path.insert(0, '.')
import oracle, workloads as W, paper_conf_icde_sioulasckaa19_b200 as hj
def dev(a): return torch.from_numpy(np.ascontiguousarray(a).view(np.int32 if a.dtype.itemsize == 4 else np.int64)).cuda()
for kb in (4, 8):
    for w in [W.Workload("a", 20000, 30011, "fk", keys="sparse" if kb == 4 else "k8", seed=400),
              W.Workload("b", 1 << 17, 1 << 18, "zipf", z=1.5, keys="sparse" if kb == 4 else "k8", seed=401)]:
        Rk, Rp, Sk, Sp = W.np_generate(w)
        m, c = oracle.hash_join(Rk, Rp, Sk, Sp)
        ctx = hj.Context(0, kb, kb)
        for bits in (-1, 3, 9, 14, 18):
            r = ctx.join(dev(Rk), dev(Rp), dev(Sk), dev(Sp), radix_bits=bits)
            print(kb, w.name, bits, (r.matches, r.checksum) == (m, c), flush=True)
print("ws small ok")
