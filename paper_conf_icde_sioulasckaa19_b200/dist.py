"""Multi-GPU radix join: one process per GPU, exchange over torch.distributed (NCCL on B200).

SURVEY.md §8(e) / DESIGN.md §7. Co-partitions are independent (all matches of
a partition are in the corresponding partition of the other relation), so G = 2^g ranks split
the co-partition space by g extra radix bits above the local field:

  1. hj_exchange_pack (per relation): histogram + planner + pass 1 with the pass-1 digit widened
     by the rank bits -> a send buffer grouped by destination rank, then by the local digit d1,
     plus per-destination count rows [G][2^local_bits].
  2. all_to_all_single of the count rows (equal splits), then of the tuples (split sizes =
     per-destination totals out, received row sums in).
  3. hj_join_received: pass 2 over the received (source, d1) segments, then the smem join.
  4. all_gather of (matches, checksum) as uint64 bit patterns, summed mod 2^64 on the host;
     materialized pairs stay sharded (their union is the result).

Every step on the data path runs in the CUDA library; this module only sizes buffers and issues
the collectives. `ctx` may be injected (tests drive the orchestration on CPU with gloo).

exchange="direct" (DirectExchange, hj_xd_join) is the B200-native form of steps 1-4: pass 1 of
every rank stores its tuples straight into the owning rank's receive window through CUDA-IPC
peer mappings (NVLink / NVSwitch on a multi-GPU node), so the send buffer, its re-read and the
tuple all-to-all disappear. The destination totals, the count rows and the results travel the
same way (stores into the peers' board windows ordered by system-scope release/acquire flags),
so one join is a sequence of kernel launches with a single host synchronization at the end;
the host takes part only when a receive window must grow (IPC handles re-shared).
"""
from __future__ import annotations

import dataclasses
import math

import numpy as np

M64 = (1 << 64) - 1


@dataclasses.dataclass
class DistResult:
    matches: int           # |R ⋈ S| over all ranks
    checksum: int          # sum of pair signatures over all ranks, mod 2^64 (count mode)
    local: object          # this rank's JoinResult (its co-partition range)
    sent_bytes: int        # tuple bytes this rank sent to other ranks (NVLink traffic)
    recv_tuples: tuple     # (R, S) tuples received


def _local_bits(nR_total: int, G: int) -> int:
    per = max(1, nR_total // G)
    return 0 if per <= 4096 else min(20, math.ceil(math.log2(per / 4096)))


def _reduce(res, group, dev):
    """all_gather of this rank's (matches, checksum) as uint64 bit patterns, summed mod 2^64."""
    import torch
    import torch.distributed as dist

    G = dist.get_world_size(group)
    if dist.get_backend(group) != "nccl":
        dev = "cpu"
    mine = torch.tensor(np.array([res.matches, res.checksum], dtype=np.uint64).view(np.int64), device=dev)
    parts = [torch.empty_like(mine) for _ in range(G)]
    dist.all_gather(parts, mine, group=group)
    m = c = 0
    for t in parts:
        a = t.cpu().numpy().view(np.uint64)
        m = (m + int(a[0])) & M64
        c = (c + int(a[1])) & M64
    return m, c


def _allgather_u64(arr: np.ndarray, group, dev) -> np.ndarray:
    """all_gather of a small uint64 array -> [G, *arr.shape] (device tensor under NCCL, CPU under gloo)."""
    import torch
    import torch.distributed as dist

    G = dist.get_world_size(group)
    t = torch.from_numpy(np.ascontiguousarray(arr, dtype=np.uint64).view(np.int64).ravel().copy())
    if dist.get_backend(group) == "nccl":
        t = t.to(dev)
    out = torch.empty(G * t.numel(), dtype=torch.int64, device=t.device)
    dist.all_gather_into_tensor(out, t, group=group)
    return out.cpu().numpy().view(np.uint64).reshape(G, *arr.shape)


def _a2a(out, inp, out_split, in_split, group):
    """all_to_all_single; under gloo (CPU collectives, tests) CUDA tensors travel through host copies."""
    import torch.distributed as dist

    if out.is_cuda and dist.get_backend(group) != "nccl":
        o = out.cpu()
        dist.all_to_all_single(o, inp.cpu(), out_split, in_split, group=group)
        out.copy_(o)
        return
    dist.all_to_all_single(out, inp, out_split, in_split, group=group)


class DirectExchange:
    """Direct-store exchange state of one rank (include/hj.h hj_xd_*): its context, its three
    windows (R receive, S receive, barrier flags), the peers' windows mapped into this process,
    and the replicated capacity table (every rank derives every window size from the same
    all-gathered totals, so growth decisions agree without another collective)."""

    def __init__(self, ctx, group=None, timeout_ms: int = 10000):
        import torch.distributed as dist

        from . import XD_BOARD_BYTES, XD_MAX_RANKS

        self.ctx, self.group, self.timeout_ms = ctx, group, timeout_ms
        self.G = dist.get_world_size(group)
        self.rank = dist.get_rank(group)
        if self.G > XD_MAX_RANKS:
            raise ValueError(f"direct exchange supports up to {XD_MAX_RANKS} ranks")
        self.tb = ctx.key_bytes + ctx.pay_bytes
        self.cap = np.zeros((2, self.G), dtype=np.int64)
        self.own = [0, 0, 0]
        self.peers = [[0] * self.G for _ in range(3)]
        self.mapped = set()
        self.own[2], h, _ = ctx.xd_window(2, XD_BOARD_BYTES)
        self._share({2: h}, [2])
        self.first = True

    def _share(self, mine: dict, slots):
        import torch.distributed as dist

        allh = [None] * self.G
        dist.all_gather_object(allh, mine, group=self.group)
        for j in range(self.G):
            for slot in slots:
                if j == self.rank:
                    self.peers[slot][j] = self.own[slot]
                elif slot in allh[j]:
                    old = self.peers[slot][j]
                    if old in self.mapped:
                        self.ctx.ipc_close(old)
                        self.mapped.discard(old)
                    self.peers[slot][j] = self.ctx.ipc_open(allh[j][slot])
                    self.mapped.add(self.peers[slot][j])

    def close(self):
        for p in list(self.mapped):
            try:
                self.ctx.ipc_close(p)
            except Exception:
                pass
        self.mapped.clear()

    def _grow(self, need):
        """Grow every window whose replicated capacity is below `need` [2, G] (bytes); identical
        decision on every rank (same inputs), then re-share the grown windows' handles."""
        grow = need > self.cap
        if not grow.any():
            return
        newcap = np.where(grow, need + need // 8 + 4096, self.cap)
        mine = {}
        for r in (0, 1):
            if grow[r, self.rank]:
                self.own[r], mine[r], _ = self.ctx.xd_window(r, int(newcap[r, self.rank]))
        self.cap = newcap
        self._share(mine, [r for r in (0, 1) if grow[r].any()])

    def join(self, Rk, Rp, Sk, Sp, local_bits: int, out_mode: int = 0) -> DistResult:
        """One device-driven join (hj_xd_join): no host collective on the data path; a window
        growth (first call, or inputs that outgrow the windows) costs one extra round."""
        from . import XD_REGROW

        G, rank, ctx, tb = self.G, self.rank, self.ctx, self.tb
        g = G.bit_length() - 1
        dev = Rk.device
        H = ctx.xd_header_bytes(G, local_bits)
        if self.first:
            # initial windows: the uniform share of all ranks' rows + 1/8 (one all-gather, once)
            n = _allgather_u64(np.array([Rk.numel(), Sk.numel()], dtype=np.uint64), self.group, dev)
            per = n.astype(np.int64).sum(axis=0) // G
            self._grow(np.repeat((H + 64 + per * tb)[:, None], G, axis=1))
            self.first = False
        for _ in range(4):
            rc, res, totals, (m, c) = ctx.xd_join(rank, g, Rk, Rp, Sk, Sp, local_bits, out_mode, self.peers[0],
                                                  self.peers[1], self.peers[2], self.cap, self.timeout_ms)
            if rc != XD_REGROW:
                break
            self._grow(H + 64 + totals.sum(axis=1).astype(np.int64) * tb)
        else:
            raise RuntimeError("direct exchange: windows still too small after growing")
        nin = tuple(int(totals[r, :, rank].sum()) for r in (0, 1))
        sent = sum(int(totals[r, rank].sum()) - int(totals[r, rank, rank]) for r in (0, 1)) * tb
        return DistResult(matches=m, checksum=c, local=res, sent_bytes=sent, recv_tuples=nin)


_XD = {}


def join(Rk, Rp, Sk, Sp, group=None, local_bits: int = -1, out_mode: int = 0, ctx=None,
         exchange: str = "nccl") -> DistResult:
    import torch
    import torch.distributed as dist

    G = dist.get_world_size(group)
    rank = dist.get_rank(group)
    g = G.bit_length() - 1
    if 1 << g != G:
        raise ValueError(f"world size {G} is not a power of two")
    dev = Rk.device
    if ctx is None:
        from . import context

        ctx = context(dev.index or 0, Rk.element_size(), Rp.element_size())
    tb = Rk.element_size() + Rp.element_size()
    words_per_tuple = tb // 8
    if local_bits < 0:
        n = torch.tensor([Rk.numel()], dtype=torch.int64, device=dev)
        dist.all_reduce(n, group=group)
        local_bits = _local_bits(int(n.item()), G)
    if exchange == "direct":
        key = (id(ctx), id(group))
        if key not in _XD:
            _XD[key] = DirectExchange(ctx, group)
        return _XD[key].join(Rk, Rp, Sk, Sp, local_bits, out_mode)
    if exchange != "nccl":
        raise ValueError(f"exchange must be 'nccl' or 'direct', not {exchange!r}")

    recv = []
    sent = 0
    for rel, (k, p) in enumerate(((Rk, Rp), (Sk, Sp))):
        send, cnt, dest = ctx.exchange_pack(rel, k, p, g, local_bits)
        cnt_recv = torch.empty_like(cnt)
        _a2a(cnt_recv, cnt, None, None, group)
        in_split = [int(x) * words_per_tuple for x in dest]
        out_tuples = [int(x) for x in cnt_recv.view(G, -1).to(torch.int64).sum(1).tolist()]
        out_split = [x * words_per_tuple for x in out_tuples]
        buf = torch.empty(sum(out_split), dtype=torch.int64, device=dev)
        _a2a(buf, send[: sum(in_split)], out_split, in_split, group)
        sent += (sum(int(x) for x in dest) - int(dest[rank])) * tb
        recv.append((buf, sum(out_tuples), cnt_recv.contiguous()))
    (rb, nr, rc), (sb, ns, sc) = recv
    res = ctx.join_received(rb, nr, rc, sb, ns, sc, G, local_bits, out_mode)
    m, c = _reduce(res, group, dev)
    return DistResult(matches=m, checksum=c, local=res, sent_bytes=sent, recv_tuples=(nr, ns))
