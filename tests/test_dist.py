"""Multi-GPU exchange path.

* CPU (`-m "not gpu"`): world_size-2 gloo run of paper_conf_icde_sioulasckaa19_b200.dist.join
  with a numpy stand-in for the CUDA library (test-only; it implements the documented layout
  of hj_exchange_pack / hj_join_received and joins with the oracle). This pins the host-side
  orchestration: rank routing, count exchange, split sizes, result reduction.
* GPU (`-m gpu`): the real exchange kernels on one device with G virtual ranks, the all-to-all
  done by slicing, checked against the oracle.
"""
import os
import socket
import types

import numpy as np
import pytest
import torch

import oracle
import workloads as W

M64 = (1 << 64) - 1


# ------------------------------------------------------------------------------------------------
# numpy stand-in of the library's exchange contract (include/hj.h), test infrastructure only
# ------------------------------------------------------------------------------------------------
class NumpyExchangeCtx:
    def __init__(self):
        self.sent_rows = {}

    @staticmethod
    def _split(lb):
        return (lb + 1) // 2, lb // 2

    def exchange_pack(self, rel, keys, pays, gpu_bits, local_bits):
        k = keys.numpy().view(np.uint32).astype(np.uint64)
        p = pays.numpy().view(np.uint32).astype(np.uint64)
        G = 1 << gpu_bits
        b1, b2 = self._split(local_bits)
        j = (k >> np.uint64(local_bits)) & np.uint64(G - 1)
        d1 = k & np.uint64((1 << b1) - 1)
        d2 = (k >> np.uint64(b1)) & np.uint64((1 << b2) - 1)
        order = np.lexsort((d1, j))  # grouped by destination, then by d1
        words = (k | (p << np.uint64(32)))[order].view(np.int64)
        q = (d1 << np.uint64(b2)) | d2
        cnt = np.zeros((G, 1 << local_bits), dtype=np.int64)
        np.add.at(cnt, (j.astype(np.int64), q.astype(np.int64)), 1)
        dest = np.bincount(j.astype(np.int64), minlength=G).astype(np.uint64)
        return torch.from_numpy(words.copy()), torch.from_numpy(cnt.astype(np.int32)), dest

    def join_received(self, R_recv, nR, R_counts, S_recv, nS, S_counts, nsrc, local_bits, out_mode=0):
        b1, b2 = self._split(local_bits)
        cols = []
        for buf, n, cnt in ((R_recv, nR, R_counts), (S_recv, nS, S_counts)):
            w = buf.numpy().view(np.uint64)
            assert len(w) == n
            k = (w & np.uint64(0xFFFFFFFF)).astype(np.uint32)
            p = (w >> np.uint64(32)).astype(np.uint32)
            # the received count rows describe the received segments exactly
            c = cnt.numpy().astype(np.int64)
            pos = 0
            for s in range(nsrc):
                seg = k[pos:pos + c[s].sum()].astype(np.uint64)
                q = ((seg & np.uint64((1 << b1) - 1)) << np.uint64(b2)) | ((seg >> np.uint64(b1)) & np.uint64((1 << b2) - 1))
                assert np.array_equal(np.bincount(q.astype(np.int64), minlength=1 << local_bits), c[s])
                pos += c[s].sum()
            assert pos == n
            cols += [k, p]
        m, chk = oracle.hash_join(*cols)
        return types.SimpleNamespace(matches=m, checksum=chk)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    return port


def _worker(rank, world, port, cfg, out):
    import torch.distributed as dist

    from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    w = W.Workload(**cfg)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    # inputs start row-sharded: rank r holds rows [r n / G, (r+1) n / G) of both relations
    rs = slice(rank * w.nR // world, (rank + 1) * w.nR // world)
    ss = slice(rank * w.nS // world, (rank + 1) * w.nS // world)
    cols = [torch.from_numpy(a[sl].view(np.int32).copy()) for a, sl in ((Rk, rs), (Rp, rs), (Sk, ss), (Sp, ss))]
    res = hjdist.join(*cols, local_bits=cfg.get("radix_bits", 6), ctx=NumpyExchangeCtx())
    out[rank] = (res.matches, res.checksum, res.local.matches, res.recv_tuples)
    dist.destroy_process_group()


@pytest.mark.parametrize("cfg", [dict(name="d1", nR=1 << 13, nS=1 << 14, dist="fk", keys="sparse", seed=130, radix_bits=6),
                                 dict(name="d2", nR=5000, nS=9000, dist="zipf", z=1.2, seed=131, radix_bits=5),
                                 dict(name="d3", nR=1 << 12, nS=1 << 12, dist="1to1", seed=132, radix_bits=4)])
def test_gloo_world2_exchange_matches_oracle(cfg):
    import multiprocessing as mp

    ctx = mp.get_context("spawn")
    mgr = ctx.Manager()
    out = mgr.dict()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, 2, port, cfg, out)) for r in range(2)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(120)
        assert p.exitcode == 0
    w = W.Workload(**{k: v for k, v in cfg.items()})
    m, c = oracle.hash_join(*W.np_generate(w))
    for r in range(2):
        assert out[r][:2] == (m, c)
    # the ranks' shares partition the result
    assert out[0][2] + out[1][2] == m
    assert out[0][2] > 0 and out[1][2] > 0


def test_local_bits_choice():
    from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist

    assert hjdist._local_bits(1 << 27, 8) == 12  # c3 at 8 GPUs: 2^24 R tuples per rank / 4096
    assert hjdist._local_bits(1 << 27, 1) == 15
    assert hjdist._local_bits(1000, 2) == 0


# ------------------------------------------------------------------------------------------------
# GPU: the real exchange kernels, G virtual ranks on one device
# ------------------------------------------------------------------------------------------------
def _virtual_exchange(hj, w, G, lb, out_mode):
    Rk, Rp, Sk, Sp = W.np_generate(w)
    g = G.bit_length() - 1
    shards = []
    for v in range(G):
        rs = slice(v * w.nR // G, (v + 1) * w.nR // G)
        ss = slice(v * w.nS // G, (v + 1) * w.nS // G)
        shards.append([torch.from_numpy(a[sl].view(np.int32).copy()).cuda() for a, sl in
                       ((Rk, rs), (Rp, rs), (Sk, ss), (Sp, ss))])
    ctx = hj.Context(0, 4, 4)
    sent = {}  # (v, rel) -> (send words clone, counts clone, dest)
    for v in range(G):
        for rel in (0, 1):
            k, p = shards[v][2 * rel], shards[v][2 * rel + 1]
            send, cnt, dest = ctx.exchange_pack(rel, k, p, g, lb)
            sent[(v, rel)] = (send.clone(), cnt.clone(), dest.copy())
    tot_m, tot_c, pairs = 0, 0, []
    for r in range(G):
        recv = []
        for rel in (0, 1):
            bufs, rows = [], []
            for s in range(G):
                words, cnt, dest = sent[(s, rel)]
                a = int(dest[:r].sum())
                bufs.append(words[a:a + int(dest[r])])
                rows.append(cnt[r])
            buf = torch.cat(bufs).contiguous()
            recv.append((buf, buf.numel(), torch.stack(rows).contiguous()))
        (rb, nr, rc), (sb, ns, sc) = recv
        res = ctx.join_received(rb, nr, rc, sb, ns, sc, G, lb, out_mode)
        torch.cuda.synchronize()
        tot_m += res.matches
        tot_c = (tot_c + res.checksum) & M64
        if out_mode == 1 and res.matches:
            pairs.append(np.stack([res.r_pay.cpu().numpy().view(np.uint32), res.s_pay.cpu().numpy().view(np.uint32)], 1))
    return (Rk, Rp, Sk, Sp), tot_m, tot_c, pairs


@pytest.mark.gpu
@pytest.mark.parametrize("G", [1, 2, 4, 8])
@pytest.mark.parametrize("dist_", ["fk", "zipf"])
def test_gpu_virtual_ranks_exchange(G, dist_):
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("v", 1 << 16, 3 << 16, dist_, keys="sparse", z=1.0, seed=140)
    for lb in (0, 5, 10):
        cols, m, c, _ = _virtual_exchange(hj, w, G, lb, 0)
        assert (m, c) == oracle.hash_join(*cols)
    cols, m, _, pairs = _virtual_exchange(hj, w, G, 8, 1)
    om, _, r, s = oracle.hash_join(*cols, materialize=True)
    assert m == om
    got = np.concatenate(pairs)
    assert np.array_equal(oracle.pairs_sorted(got[:, 0], got[:, 1]), oracle.pairs_sorted(r, s))


_NCCL1 = r'''
import os, sys, numpy as np, torch, torch.distributed as dist
sys.path.insert(0, sys.argv[1])
import oracle, workloads as W
from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist
dist.init_process_group("nccl", rank=0, world_size=1)
torch.cuda.set_device(0)
w = W.Workload("n", 1 << 16, 3 << 16, "zipf", keys="sparse", z=1.0, seed=180)
Rk, Rp, Sk, Sp = W.np_generate(w)
cols = [torch.from_numpy(a.view(np.int32)).cuda() for a in (Rk, Rp, Sk, Sp)]
for lb in (0, 6, 12):
    r = hjdist.join(*cols, local_bits=lb)
    assert (r.matches, r.checksum) == oracle.hash_join(Rk, Rp, Sk, Sp), lb
r = hjdist.join(*cols, out_mode=1)
m, c, rr, ss = oracle.hash_join(Rk, Rp, Sk, Sp, materialize=True)
got = oracle.pairs_sorted(r.local.r_pay.cpu().numpy().view(np.uint32), r.local.s_pay.cpu().numpy().view(np.uint32))
assert r.matches == m and np.array_equal(got, oracle.pairs_sorted(rr, ss))
dist.destroy_process_group()
print("nccl1 ok")
'''


@pytest.mark.gpu
def test_dist_join_nccl_one_rank():
    """dist.join through real NCCL collectives (one rank: the exchange sends everything to
    itself), against the oracle -- the plumbing bench.py --gpus N uses."""
    import subprocess
    import sys

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, MASTER_ADDR="127.0.0.1", MASTER_PORT=str(_free_port()), RANK="0", WORLD_SIZE="1",
               LOCAL_RANK="0")
    out = subprocess.run([sys.executable, "-c", _NCCL1, root], capture_output=True, text=True, timeout=600, env=env)
    assert "nccl1 ok" in out.stdout, out.stdout[-2000:] + out.stderr[-4000:]
