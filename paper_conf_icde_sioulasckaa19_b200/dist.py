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


def join(Rk, Rp, Sk, Sp, group=None, local_bits: int = -1, out_mode: int = 0, ctx=None) -> DistResult:
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

    recv = []
    sent = 0
    for rel, (k, p) in enumerate(((Rk, Rp), (Sk, Sp))):
        send, cnt, dest = ctx.exchange_pack(rel, k, p, g, local_bits)
        cnt_recv = torch.empty_like(cnt)
        dist.all_to_all_single(cnt_recv, cnt, group=group)
        in_split = [int(x) * words_per_tuple for x in dest]
        out_tuples = [int(x) for x in cnt_recv.view(G, -1).to(torch.int64).sum(1).tolist()]
        out_split = [x * words_per_tuple for x in out_tuples]
        buf = torch.empty(sum(out_split), dtype=torch.int64, device=dev)
        dist.all_to_all_single(buf, send[: sum(in_split)], out_split, in_split, group=group)
        sent += (sum(int(x) for x in dest) - int(dest[rank])) * tb
        recv.append((buf, sum(out_tuples), cnt_recv.contiguous()))
    (rb, nr, rc), (sb, ns, sc) = recv
    res = ctx.join_received(rb, nr, rc, sb, ns, sc, G, local_bits, out_mode)
    mine = torch.tensor(np.array([res.matches, res.checksum], dtype=np.uint64).view(np.int64), device=dev)
    parts = [torch.empty_like(mine) for _ in range(G)]
    dist.all_gather(parts, mine, group=group)
    m = c = 0
    for t in parts:
        a = t.cpu().numpy().view(np.uint64)
        m = (m + int(a[0])) & M64
        c = (c + int(a[1])) & M64
    return DistResult(matches=m, checksum=c, local=res, sent_bytes=sent, recv_tuples=(nr, ns))
