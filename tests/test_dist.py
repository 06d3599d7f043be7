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
    def _b1(G, lb):  # hj_exchange_row_len's rule: b1 = min(ceil(lb / 2), 10 - log2 G)
        g = G.bit_length() - 1
        b1 = (lb + 1) // 2
        return max(0, 10 - g) if g > 0 and b1 > 10 - g else b1

    def exchange_pack(self, rel, keys, pays, gpu_bits, local_bits):
        k = keys.numpy().view(np.uint32).astype(np.uint64)
        p = pays.numpy().view(np.uint32).astype(np.uint64)
        G = 1 << gpu_bits
        b1 = self._b1(G, local_bits)
        j = (k >> np.uint64(local_bits)) & np.uint64(G - 1)
        d1 = k & np.uint64((1 << b1) - 1)
        order = np.lexsort((d1, j))  # grouped by destination, then by d1
        words = (k | (p << np.uint64(32)))[order].view(np.int64)
        cnt = np.zeros((G, 1 << b1), dtype=np.int64)  # piece counts: tuples per (destination, d1)
        np.add.at(cnt, (j.astype(np.int64), d1.astype(np.int64)), 1)
        dest = np.bincount(j.astype(np.int64), minlength=G).astype(np.uint64)
        return torch.from_numpy(words.copy()), torch.from_numpy(cnt.astype(np.int32)), dest

    def join_received(self, R_recv, nR, R_counts, S_recv, nS, S_counts, nsrc, local_bits, out_mode=0):
        b1 = self._b1(nsrc, local_bits)
        cols = []
        for buf, n, cnt in ((R_recv, nR, R_counts), (S_recv, nS, S_counts)):
            w = buf.numpy().view(np.uint64)
            assert len(w) == n
            k = (w & np.uint64(0xFFFFFFFF)).astype(np.uint32)
            p = (w >> np.uint64(32)).astype(np.uint32)
            # the received piece rows describe the received segments exactly (source-major, d1-grouped)
            c = cnt.numpy().astype(np.int64)
            pos = 0
            for s in range(nsrc):
                for d in range(1 << b1):
                    seg = k[pos:pos + c[s, d]].astype(np.uint64)
                    assert np.all((seg & np.uint64((1 << b1) - 1)) == np.uint64(d))
                    pos += c[s, d]
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


class NumpyDirectCtx(NumpyExchangeCtx):
    """Stand-in of the direct-store contract (include/hj.h hj_xd_*), test infrastructure only:
    windows are POSIX shared-memory segments (the 64-byte "IPC handle" is the segment name), so
    the stores of one process really land in another's window with the documented layout
    (count-row header, then tuples source-major, each source's run grouped by d1)."""

    key_bytes = pay_bytes = 4

    def __init__(self):
        super().__init__()
        self.seg = {}      # fake device address -> SharedMemory
        self.next = 1 << 40
        self.own = {}      # slot -> address
        self.grew_log = []

    def _add(self, shm):
        a = self.next
        self.next += 1 << 36
        self.seg[a] = shm
        return a

    def _buf(self, addr):
        base = max(a for a in self.seg if a <= addr)
        return np.ndarray((self.seg[base].size,), dtype=np.uint8, buffer=self.seg[base].buf), addr - base

    def xd_header_bytes(self, G, lb):
        return -(-G * (4 << self._b1(G, lb)) // 256) * 256

    def xd_window(self, slot, nbytes, want_handle=True):
        from multiprocessing import shared_memory

        old = self.own.get(slot)
        if old is not None and self.seg[old].size >= nbytes:
            return old, self.seg[old].name.encode().ljust(64, b"\0"), False
        shm = shared_memory.SharedMemory(create=True, size=max(int(nbytes), 256))
        shm.buf[:] = bytes(shm.size)
        self.own[slot] = self._add(shm)
        self.grew_log.append((slot, int(nbytes)))
        return self.own[slot], shm.name.encode().ljust(64, b"\0"), True

    def ipc_open(self, handle):
        from multiprocessing import shared_memory

        return self._add(shared_memory.SharedMemory(name=handle.rstrip(b"\0").decode()))

    def ipc_close(self, addr):
        self.seg.pop(addr).close()

    def _u64(self, addr, idx, n=1):
        buf, o = self._buf(addr)
        return buf[o + 8 * idx:o + 8 * (idx + n)].view(np.uint64)

    def xd_join(self, rank, g, Rk, Rp, Sk, Sp, lb, out_mode, win_R, win_S, board, win_bytes, timeout_ms=10000):
        """hj_xd_join's documented phases, with gloo barriers standing in for the flag waits."""
        import torch.distributed as dist

        G = 1 << g
        H = self.xd_header_bytes(G, lb)
        TOT, RES = 192, 192 + 64 * 2 * 64
        sent = [self.exchange_pack(r, k, p, g, lb) for r, (k, p) in enumerate(((Rk, Rp), (Sk, Sp)))]
        for j in range(G):  # phase A: totals into every board
            for r in (0, 1):
                self._u64(int(board[j]), TOT + (rank * 2 + r) * 64, G)[:] = sent[r][2]
        dist.barrier()
        own = self._u64(int(board[rank]), TOT, G * 2 * 64).reshape(G, 2, 64)[:, :, :G]
        totals = np.ascontiguousarray(own.transpose(1, 0, 2)).astype(np.uint64)   # [r, src, dst]
        cap = (np.asarray(win_bytes, dtype=np.int64).reshape(2, G) - H - 64) // 8
        over = (totals.sum(axis=1).astype(np.int64) > cap).any()
        if not over:  # count rows + tuples into the owners' windows (source-major, d1-grouped)
            for r, win in ((0, win_R), (1, win_S)):
                words, cnt, d = (x.numpy() if hasattr(x, "numpy") else x for x in sent[r])
                for j in range(G):
                    buf, o = self._buf(int(win[j]))
                    row = cnt[j].astype(np.uint32).view(np.uint8)
                    buf[o + rank * row.size:o + (rank + 1) * row.size] = row
                    a, n = int(d[:j].sum()), int(d[j])
                    base = int(totals[r, :rank, j].sum())
                    seg = words[a:a + n].view(np.uint8)
                    buf[o + H + 8 * base:o + H + 8 * base + seg.size] = seg
        dist.barrier()  # phase B
        if over:
            return 1, types.SimpleNamespace(matches=0, checksum=0), totals, (0, 0)
        ins = []
        for r, win in ((0, win_R), (1, win_S)):
            n = int(totals[r, :, rank].sum())
            buf, o = self._buf(int(win[rank]))
            rl = 1 << self._b1(G, lb)
            cnt = buf[o:o + G * 4 * rl].view(np.int32).reshape(G, rl).copy()
            recv = buf[o + H:o + H + 8 * n].view(np.int64).copy()
            ins += [torch.from_numpy(recv), n, torch.from_numpy(cnt)]
        res = self.join_received(*ins, G, lb, out_mode)
        for j in range(G):  # phase C
            self._u64(int(board[j]), RES + 2 * rank, 2)[:] = [res.matches, res.checksum]
        dist.barrier()
        allr = self._u64(int(board[rank]), RES, 2 * G).reshape(G, 2).astype(object).sum(axis=0)
        dist.barrier()  # every rank read its board before the next call's phase A
        return 0, res, totals, (int(allr[0]) & M64, int(allr[1]) & M64)

    def close(self):
        for a in list(self.seg):
            shm = self.seg.pop(a)
            shm.close()
            if a in self.own.values():
                shm.unlink()


def _direct_worker(rank, world, port, out):
    import torch.distributed as dist

    from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist

    os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
    dist.init_process_group("gloo", rank=rank, world_size=world)
    ctx = NumpyDirectCtx()
    xd = hjdist.DirectExchange(ctx)
    res = []
    # growing inputs: the windows must grow (and be re-shared) on the second and third call
    for i, (nR, nS, lb, dist_) in enumerate([(1 << 11, 1 << 12, 4, "fk"), (1 << 13, 1 << 14, 6, "zipf"),
                                             (3000, 20000, 5, "zipf"), (1 << 12, 1 << 12, 6, "1to1")]):
        w = W.Workload("dx", nR, nS, dist_, keys="sparse", z=1.3, seed=150 + i)
        Rk, Rp, Sk, Sp = W.np_generate(w)
        rs = slice(rank * nR // world, (rank + 1) * nR // world)
        ss = slice(rank * nS // world, (rank + 1) * nS // world)
        cols = [torch.from_numpy(a[sl].view(np.int32).copy()) for a, sl in ((Rk, rs), (Rp, rs), (Sk, ss), (Sp, ss))]
        r = xd.join(*cols, local_bits=lb)
        res.append((r.matches, r.checksum, r.local.matches, r.recv_tuples, r.sent_bytes))
    out[rank] = (res, list(ctx.grew_log))
    xd.close()
    dist.barrier()
    ctx.close()
    dist.destroy_process_group()


def test_gloo_world2_direct_exchange_matches_oracle():
    """DirectExchange orchestration across two processes (gloo): totals all-gather, replicated
    window capacities, growth + handle re-exchange, source-major window layout, reduction."""
    import multiprocessing as mp

    ctx = mp.get_context("spawn")
    mgr = ctx.Manager()
    out = mgr.dict()
    port = _free_port()
    procs = [ctx.Process(target=_direct_worker, args=(r, 2, port, out)) for r in range(2)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(180)
        assert p.exitcode == 0
    for i, (nR, nS, lb, dist_) in enumerate([(1 << 11, 1 << 12, 4, "fk"), (1 << 13, 1 << 14, 6, "zipf"),
                                             (3000, 20000, 5, "zipf"), (1 << 12, 1 << 12, 6, "1to1")]):
        w = W.Workload("dx", nR, nS, dist_, keys="sparse", z=1.3, seed=150 + i)
        m, c = oracle.hash_join(*W.np_generate(w))
        for r in range(2):
            assert out[r][0][i][:2] == (m, c), (i, r)
        assert out[0][0][i][2] + out[1][0][i][2] == m
        assert sum(out[r][0][i][3][0] for r in range(2)) == nR and sum(out[r][0][i][3][1] for r in range(2)) == nS
    # windows grew at least once after the first call (re-shared handles were used)
    assert any(len([g for g in out[r][1] if g[0] in (0, 1)]) > 2 for r in range(2))


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
def test_gpu_join_received_rejects_inconsistent_counts():
    """hj_join_received sizes its buffers from nR / nS: count rows that describe more tuples than
    that must fail (HJ_ERR_INVALID) without writing out of bounds, and the same
    context must give the right result on the next, consistent call."""
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("bad", 20000, 30000, "fk", keys="sparse", seed=133)
    Rk, Rp, Sk, Sp = W.np_generate(w)
    ctx = hj.Context(0, 4, 4)
    packed = []
    for rel, (k, p) in enumerate(((Rk, Rp), (Sk, Sp))):
        send, cnt, dest = ctx.exchange_pack(rel, torch.from_numpy(k.view(np.int32)).cuda(),
                                            torch.from_numpy(p.view(np.int32)).cuda(), 0, 7)
        packed.append((send.clone(), cnt.clone()))
    (rs, rc), (ss, sc) = packed
    with pytest.raises(hj.HJError, match="INVALID"):
        ctx.join_received(rs, w.nR - 1000, rc, ss, w.nS, sc, 1, 7)
    res = ctx.join_received(rs, w.nR, rc, ss, w.nS, sc, 1, 7)
    assert (res.matches, res.checksum) == oracle.hash_join(Rk, Rp, Sk, Sp)
    ctx.close()


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


# ------------------------------------------------------------------------------------------------
# GPU: direct-store exchange (hj_xd_*), pass 1 writing straight into the owners' windows
# ------------------------------------------------------------------------------------------------
def _direct_virtual(hj, w, G, lb, out_mode, width=4):
    """G virtual ranks in one process, one context and one CUDA stream each; every rank's
    windows are plain device pointers here (same process: no IPC mapping), the barrier kernels
    of the G streams run concurrently."""
    cols = W.np_generate(w)
    g = G.bit_length() - 1
    view = np.int32 if width == 4 else np.int64
    shards = []
    for v in range(G):
        rs = slice(v * w.nR // G, (v + 1) * w.nR // G)
        ss = slice(v * w.nS // G, (v + 1) * w.nS // G)
        shards.append([torch.from_numpy(a[sl].view(view).copy()).cuda() for a, sl in
                       zip(cols, (rs, rs, ss, ss))])
    ctxs = [hj.Context(0, width, width) for _ in range(G)]
    streams = [torch.cuda.Stream() for _ in range(G)]
    torch.cuda.synchronize()
    dest = []
    for v in range(G):
        with torch.cuda.stream(streams[v]):
            dest.append(ctxs[v].xd_count(*shards[v], g, lb))
    totals = np.ascontiguousarray(np.stack(dest).transpose(1, 0, 2))  # [2, src, dst]
    H = hj.xd_header_bytes(G, lb)
    tb = 2 * width
    win = [[0] * G for _ in range(3)]
    for v in range(G):
        for r in (0, 1):
            win[r][v], _, _ = ctxs[v].xd_window(r, H + int(totals[r, :, v].sum()) * tb + 64, want_handle=False)
        win[2][v], _, _ = ctxs[v].xd_window(2, 8 * 64, want_handle=False)
    for v in range(G):
        with torch.cuda.stream(streams[v]):
            ctxs[v].xd_store(v, totals, win[0], win[1])
    for v in range(G):
        with torch.cuda.stream(streams[v]):
            ctxs[v].xd_barrier(v, win[2], 20000)
    tot_m, tot_c, pairs = 0, 0, []
    for v in range(G):
        nin = [int(totals[r, :, v].sum()) for r in (0, 1)]
        ins = []
        for r in (0, 1):
            words = nin[r] * tb // 8
            recv = hj._wrap_device(win[r][v] + H, max(words, 1), 8, torch.device("cuda", 0))[:words]
            rl = hj.exchange_row_len(G, lb)
            cnt = hj._wrap_device(win[r][v], G * rl, 4, torch.device("cuda", 0)).view(G, rl)
            ins += [recv, nin[r], cnt]
        with torch.cuda.stream(streams[v]):
            res = ctxs[v].join_received(*ins, G, lb, out_mode)
        tot_m += res.matches
        tot_c = (tot_c + res.checksum) & M64
        if out_mode == 1 and res.matches:
            pv = np.uint32 if width == 4 else np.uint64
            pairs.append(np.stack([res.r_pay.cpu().numpy().view(pv), res.s_pay.cpu().numpy().view(pv)], 1))
    torch.cuda.synchronize()
    for c in ctxs:
        c.close()
    return cols, tot_m, tot_c, pairs


@pytest.mark.gpu
@pytest.mark.parametrize("G", [1, 2, 4, 8])
@pytest.mark.parametrize("dist_", ["fk", "zipf"])
def test_gpu_direct_store_virtual_ranks(G, dist_):
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("x", 1 << 16, 3 << 16, dist_, keys="sparse", z=1.0, seed=190)
    for lb in (0, 5, 10):
        cols, m, c, _ = _direct_virtual(hj, w, G, lb, 0)
        assert (m, c) == oracle.hash_join(*cols), lb
    cols, m, _, pairs = _direct_virtual(hj, w, G, 8, 1)
    om, _, r, s = oracle.hash_join(*cols, materialize=True)
    assert m == om
    got = np.concatenate(pairs)
    assert np.array_equal(oracle.pairs_sorted(got[:, 0], got[:, 1]), oracle.pairs_sorted(r, s))


@pytest.mark.gpu
@pytest.mark.parametrize("G", [2, 8])
def test_gpu_direct_store_8byte_and_ragged(G):
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("x8", 50001, 77777, "fk", keys="k8", seed=191)
    cols, m, c, _ = _direct_virtual(hj, w, G, 7, 0, width=8)
    assert (m, c) == oracle.hash_join(*cols)


_XD2 = r'''
import os, sys, numpy as np, torch, torch.distributed as dist
sys.path.insert(0, sys.argv[1])
import oracle, workloads as W
from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist
rank, G = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
dist.init_process_group("gloo", rank=rank, world_size=G)
torch.cuda.set_device(0)
for i, (nR, nS, lb, mode) in enumerate([(1 << 14, 1 << 15, 6, 0), (1 << 16, 3 << 16, 9, 0), (5000, 9000, 4, 1),
                                        (1 << 16, 3 << 16, 9, 1)]):
    w = W.Workload("x", nR, nS, "zipf", keys="sparse", z=1.0, seed=200 + i)
    cols = W.np_generate(w)
    rs = slice(rank * nR // G, (rank + 1) * nR // G)
    ss = slice(rank * nS // G, (rank + 1) * nS // G)
    mine = [torch.from_numpy(a[sl].view(np.int32).copy()).cuda() for a, sl in zip(cols, (rs, rs, ss, ss))]
    r = hjdist.join(*mine, local_bits=lb, out_mode=mode, exchange="direct")
    m, c = oracle.hash_join(*cols)
    assert r.matches == m, (i, r.matches, m)
    if mode == 0:
        assert r.checksum == c, i
    else:  # the ranks' materialized shares partition the pairs
        got = np.stack([r.local.r_pay.cpu().numpy().view(np.uint32), r.local.s_pay.cpu().numpy().view(np.uint32)], 1)
        allp = [None] * G
        dist.all_gather_object(allp, got)
        allp = np.concatenate(allp)
        _, _, rr, sp = oracle.hash_join(*cols, materialize=True)
        assert np.array_equal(oracle.pairs_sorted(allp[:, 0], allp[:, 1]), oracle.pairs_sorted(rr, sp)), i
dist.destroy_process_group()
print("xd2 ok", rank)
'''


@pytest.mark.gpu
def test_direct_exchange_two_processes_one_gpu():
    """dist.join(exchange='direct') across two PROCESSES sharing one B200: windows exported and
    opened through CUDA IPC, pass-1 stores into the other process's window, the device flag
    barrier across contexts (time-sliced on one GPU), window growth and handle re-exchange."""
    import subprocess
    import sys

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    port = str(_free_port())
    procs = []
    for r in range(2):
        env = dict(os.environ, MASTER_ADDR="127.0.0.1", MASTER_PORT=port, RANK=str(r), WORLD_SIZE="2")
        procs.append(subprocess.Popen([sys.executable, "-c", _XD2, root], stdout=subprocess.PIPE,
                                      stderr=subprocess.PIPE, text=True, env=env))
    outs = [p.communicate(timeout=600) for p in procs]
    for r, (o, e) in enumerate(outs):
        assert f"xd2 ok {r}" in o, o[-2000:] + e[-4000:]


def _xd_join_threads(hj, w, G, lb, out_mode, width=4, calls=2, cap_scale=1.0):
    """hj_xd_join with G virtual ranks in one process: one host thread, context and CUDA stream
    per rank (the call is synchronous and its phase waits need every rank's kernels running)."""
    import concurrent.futures as cf

    cols = W.np_generate(w)
    g = G.bit_length() - 1
    view = np.int32 if width == 4 else np.int64
    shards = []
    for v in range(G):
        rs = slice(v * w.nR // G, (v + 1) * w.nR // G)
        ss = slice(v * w.nS // G, (v + 1) * w.nS // G)
        shards.append([torch.from_numpy(a[sl].view(view).copy()).cuda() for a, sl in zip(cols, (rs, rs, ss, ss))])
    ctxs = [hj.Context(0, width, width) for _ in range(G)]
    streams = [torch.cuda.Stream() for _ in range(G)]
    H = hj.xd_header_bytes(G, lb)
    tb = 2 * width
    cap = np.zeros((2, G), dtype=np.uint64)
    win = [[0] * G for _ in range(3)]
    for v in range(G):
        for r, n in ((0, w.nR), (1, w.nS)):
            cap[r, v] = H + 64 + int(cap_scale * n / G + 16) * tb
            win[r][v], _, _ = ctxs[v].xd_window(r, int(cap[r, v]), want_handle=False)
        win[2][v], _, _ = ctxs[v].xd_window(2, hj.XD_BOARD_BYTES, want_handle=False)
    for v in range(G):  # ranks share this GPU: no allocation may run while a peer's kernels wait
        ctxs[v].xd_reserve(g, shards[v][0].numel(), shards[v][2].numel(), lb, out_mode, cap[0, v], cap[1, v])
    torch.cuda.synchronize()

    def rank_call(v):
        with torch.cuda.stream(streams[v]):
            out = ctxs[v].xd_join(v, g, *shards[v], lb, out_mode, win[0], win[1], win[2], cap, 20000)
            if out[1].r_pay is not None:
                pv = np.uint32 if width == 4 else np.uint64
                out = out + (np.stack([out[1].r_pay.cpu().numpy().view(pv), out[1].s_pay.cpu().numpy().view(pv)], 1),)
            return out

    results = []
    with cf.ThreadPoolExecutor(G) as ex:
        for _ in range(calls):
            results.append(list(ex.map(rank_call, range(G))))
    torch.cuda.synchronize()
    for c in ctxs:
        c.close()
    return cols, results


@pytest.mark.gpu
@pytest.mark.parametrize("G", [1, 2, 4, 8])
@pytest.mark.parametrize("dist_", ["fk", "zipf"])
def test_gpu_xd_join_virtual_ranks(G, dist_):
    """hj_xd_join (device-driven exchange: totals, count rows, tuples and results through peer
    boards / windows) against the oracle, repeated calls on the same windows."""
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("xj", 1 << 16, 3 << 16, dist_, keys="sparse", z=1.0, seed=195)
    for lb, mode in ((0, 0), (6, 0), (10, 0), (8, 1)):
        cols, calls = _xd_join_threads(hj, w, G, lb, mode, cap_scale=4.0)  # zipf: the hot rank gets > 1/G
        m, c, rr, ss = oracle.hash_join(*cols, materialize=True)
        for outs in calls:
            assert all(o[0] == 0 for o in outs)
            assert sum(o[1].matches for o in outs) == m
            for o in outs:
                assert o[3][0] == m
                if mode == 0:
                    assert o[3][1] == c
            tot = outs[0][2]
            assert all(np.array_equal(o[2], tot) for o in outs)
            assert int(tot[0].sum()) == w.nR and int(tot[1].sum()) == w.nS
            if mode == 1:
                got = np.concatenate([o[4] for o in outs if len(o) > 4])
                assert np.array_equal(oracle.pairs_sorted(got[:, 0], got[:, 1]), oracle.pairs_sorted(rr, ss))


@pytest.mark.gpu
def test_gpu_xd_join_regrow_and_8byte():
    """Windows too small: every rank returns HJ_XD_REGROW in the same call with the totals that
    size them, and nothing was joined; 8-byte tuples."""
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("xr", 1 << 15, 1 << 16, "zipf", keys="sparse", z=1.5, seed=196)
    cols, calls = _xd_join_threads(hj, w, 4, 6, 0, calls=1, cap_scale=0.5)
    outs = calls[0]
    assert all(o[0] == hj.XD_REGROW for o in outs)
    tot = outs[0][2]
    assert int(tot[0].sum()) == w.nR and int(tot[1].sum()) == w.nS
    w8 = W.Workload("x8", 40000, 70001, "fk", keys="k8", seed=197)
    cols, calls = _xd_join_threads(hj, w8, 4, 7, 0, width=8, cap_scale=2.0)
    m, c = oracle.hash_join(*cols)
    for outs in calls:
        assert all(o[0] == 0 and o[3] == (m, c) for o in outs)


@pytest.mark.gpu
@pytest.mark.parametrize("G,lb", [(8, 16), (4, 17), (2, 18)])
def test_gpu_exchange_c5_local_bits(G, lb):
    """The local radix bits c5 needs at G = 2/4/8 (2^31 rows: 18/17/16 bits): the pass-1 fan-out
    (rank bits + b1) and the receiver's pieces stay <= 2^10 by b1 = min(ceil(B/2), 10 - log2 G),
    on both exchange paths, 8-byte tuples."""
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("c5s", 1 << 15, 1 << 15, "1to1", keys="k8", seed=198)
    cols, calls = _xd_join_threads(hj, w, G, lb, 0, width=8, calls=1, cap_scale=2.0)
    m, c = oracle.hash_join(*cols)
    assert all(o[0] == 0 and o[3] == (m, c) for o in calls[0])


@pytest.mark.gpu
@pytest.mark.slow
def test_gpu_xd_join_c5_bits_at_scale():
    """c5's multi-GPU shape at scale: G = 8 virtual ranks, local_bits = 16, 8-byte 1:1 keys,
    2^23 rows of R and of S per rank (2^26 each): every rank's all-rank result equals the closed
    form (|S| matches, checksum = sum_j sig(rho(j), j))."""
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("c5x", 1 << 26, 1 << 26, "1to1", keys="k8", seed=108)
    cols, calls = _xd_join_threads(hj, w, 8, 16, 0, width=8, calls=2, cap_scale=1.25)
    j = np.arange(w.nS, dtype=np.uint64)
    rho = W.np_rho_for(w, j)
    with np.errstate(over="ignore"):
        exp = int(W.np_fmix64(rho ^ (j * np.uint64(0x9E3779B97F4A7C15))).sum(dtype=np.uint64))
    for outs in calls:
        assert all(o[0] == 0 and o[3] == (w.nS, exp) for o in outs), [o[:1] + o[3:4] for o in outs]


@pytest.mark.gpu
@pytest.mark.parametrize("nR,nS", [(3, 5000), (5000, 2), (1, 1)])
def test_gpu_xd_join_ranks_without_rows(nR, nS):
    """A rank with no local rows of R or S still takes part in every phase of hj_xd_join (its
    peers wait on its flags): tiny relations over 4 virtual ranks."""
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    import paper_conf_icde_sioulasckaa19_b200 as hj

    w = W.Workload("tiny", nR, nS, "fk", keys="sparse", seed=199)
    cols, calls = _xd_join_threads(hj, w, 4, 2, 0, calls=2, cap_scale=8.0)
    m, c = oracle.hash_join(*cols)
    for outs in calls:
        assert all(o[0] == 0 and o[3] == (m, c) for o in outs)
