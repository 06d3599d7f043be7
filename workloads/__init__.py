"""Seeded, counter-based synthetic workload generators.

This module is shared by the oracle harness and the CUDA harness and holds
NONE of the join's arithmetic: it only produces input columns (and, for
closed-form pins, the row map rho that the generator itself chose).

Two bit-identical implementations of the same integer definitions:
  * ``np_*``    numpy uint64 (host; used for oracle inputs),
  * ``torch_*`` torch int64 with wrap-around arithmetic (host or CUDA; used to
    create large inputs directly in HBM).
``tests/test_workloads.py`` checks both agree bit for bit.

Workload of the paper (§V-A): two narrow columnar tables,
each a 4-byte key and a 4-byte value; keys "unique and uniform"
(PAPER.md:681-682). Probe-side ratios 1:k with "the same set of distinct
values"; Zipf-skewed probe keys (PAPER.md:1288-1300,
Fig. 17). Readings S14-S16 of SURVEY.md §8(c.4) fix what the paper leaves
open; DESIGN.md lists them.

Definitions (all arithmetic mod 2^64 unless stated):
  fmix64(z)            splitmix64 finalizer
  rng(seed, tag, i)    fmix64(fmix64(seed ^ tag) + i * GOLDEN)
  perm(seed, k, x)     4-round bijection on [0, 2^k):
                         x = (x + c_r) mod 2^k; x ^= x >> ceil(k/2); x = x * a_r mod 2^k
                       c_r = fmix64(seed ^ (0x100 + r)), a_r = fmix64(seed ^ (0x200 + r)) | 1
  perm_n(seed, n, x)   cycle-walking restriction of perm(seed, ceil(log2 n)) to [0, n)
  key maps             dense4: x + 1;  sparse4: fmix32(x + 1);  k8: fmix64((x + 1) ^ seed_k)
  R                    R_key[i] = K(perm_n(seed_R, nR, i)), R_pay[i] = i
  S                    S_key[j] = R_key[rho(j)], S_pay[j] = j
  NEXT-2 skew / duplicate workloads (Fig. 17 build-side and identical skew, Fig. 19 replicas):
    'zipf_build': R_key[i] = K(perm_n(seed_Z, nS, zrank(seed,'B',i; nS))), S_key[j] = K(perm_n(seed_S, nS, j))
    'zipf_both' : R_key[i] = K(perm_n(seed_Z, nR, zrank(seed,'B',i; nR))), S_key[j] = K(perm_n(seed_Z, nR, zrank(seed,'Z',j; nR)))
    'replicas'  : R_key[i] = K(perm_n(seed_R, nR, i) mod D), S_key[j] = K(perm_n(seed_S, nS, j) mod D), D = nR / rep
  rho                  'fk'   : mulhi32(rng(seed,'U',j) >> 32, nR)  (== rng >> (64-log2 nR) for 2^k)
                       '1to1' : perm_n(seed_S, nS, j)  (nS == nR)
                       'zipf' : perm_n(seed_Z, nR, rank_j), rank_j = first k with CDF[k] >= u_j*CDF[-1]
                                u_j = (rng(seed,'Z',j) >> 11) * 2^-53, CDF[k] = cumsum((t+1)^-z) (host, float64,
                                sequential accumulation, shipped as the same bytes to the device)
"""
from __future__ import annotations

import dataclasses
import math

import numpy as np

GOLDEN = 0x9E3779B97F4A7C15
M64 = (1 << 64) - 1

TAG_R = 0x52  # 'R'
TAG_S = 0x53  # 'S'
TAG_Z = 0x5A  # 'Z'
TAG_U = 0x55  # 'U'
TAG_K = 0x4B  # 'K'
TAG_B = 0x42  # 'B'


# ----------------------------------------------------------------------------------------------
# scalar (python int) reference of the generator primitives, used for seed derivation
# ----------------------------------------------------------------------------------------------
def fmix64_int(z: int) -> int:
    z &= M64
    z ^= z >> 30
    z = (z * 0xBF58476D1CE4E5B9) & M64
    z ^= z >> 27
    z = (z * 0x94D049BB133111EB) & M64
    z ^= z >> 31
    return z


def sub_seed(seed: int, tag: int) -> int:
    return fmix64_int((seed ^ (tag << 56)) & M64)


def perm_constants(seed: int):
    cs = [fmix64_int(seed ^ (0x100 + r)) for r in range(4)]
    as_ = [fmix64_int(seed ^ (0x200 + r)) | 1 for r in range(4)]
    return cs, as_


# ----------------------------------------------------------------------------------------------
# numpy implementation (uint64, wraps mod 2^64)
# ----------------------------------------------------------------------------------------------
def np_fmix64(z: np.ndarray) -> np.ndarray:
    z = z.astype(np.uint64, copy=True)
    z ^= z >> np.uint64(30)
    z *= np.uint64(0xBF58476D1CE4E5B9)
    z ^= z >> np.uint64(27)
    z *= np.uint64(0x94D049BB133111EB)
    z ^= z >> np.uint64(31)
    return z


def np_fmix32(h: np.ndarray) -> np.ndarray:
    h = h.astype(np.uint32, copy=True)
    h ^= h >> np.uint32(16)
    h *= np.uint32(0x85EBCA6B)
    h ^= h >> np.uint32(13)
    h *= np.uint32(0xC2B2AE35)
    h ^= h >> np.uint32(16)
    return h


def np_rng(seed: int, tag: int, idx: np.ndarray) -> np.ndarray:
    base = np.uint64(fmix64_int(seed ^ tag))
    with np.errstate(over="ignore"):
        return np_fmix64(base + idx.astype(np.uint64) * np.uint64(GOLDEN))


def _bits_for(n: int) -> int:
    return max(0, (n - 1).bit_length())


def np_perm_pow2(seed: int, k: int, x: np.ndarray) -> np.ndarray:
    """Bijection on [0, 2^k)."""
    x = x.astype(np.uint64, copy=True)
    if k == 0:
        return np.zeros_like(x)
    mask = np.uint64((1 << k) - 1)
    sh = np.uint64((k + 1) // 2)
    cs, as_ = perm_constants(seed)
    with np.errstate(over="ignore"):
        for r in range(4):
            x = (x + np.uint64(cs[r])) & mask
            x ^= x >> sh
            x = (x * np.uint64(as_[r])) & mask
    return x


def np_perm_n(seed: int, n: int, x: np.ndarray) -> np.ndarray:
    """Bijection on [0, n) by cycle walking over the next power of two."""
    k = _bits_for(n)
    y = np_perm_pow2(seed, k, x)
    if n == (1 << k):
        return y
    bad = y >= np.uint64(n)
    while bad.any():
        y[bad] = np_perm_pow2(seed, k, y[bad])
        bad = y >= np.uint64(n)
    return y


def np_keymap(kind: str, x: np.ndarray, seed: int) -> np.ndarray:
    x = x.astype(np.uint64)
    if kind == "dense":
        return (x + np.uint64(1)).astype(np.uint32)
    if kind == "sparse":
        return np_fmix32((x + np.uint64(1)).astype(np.uint32))
    if kind == "k8":
        with np.errstate(over="ignore"):
            return np_fmix64((x + np.uint64(1)) ^ np.uint64(sub_seed(seed, TAG_K)))
    raise ValueError(kind)


def zipf_cdf(n: int, z: float) -> np.ndarray:
    """CDF[k] = sum_{t<=k} (t+1)^-z, float64, sequential accumulation (np.cumsum)."""
    w = np.power(np.arange(1, n + 1, dtype=np.float64), -float(z))
    return np.cumsum(w)


def np_zrank(seed: int, tag: int, idx: np.ndarray, cdf: np.ndarray) -> np.ndarray:
    """Zipf rank of row idx: first k with CDF[k] >= u * CDF[-1], u = (rng >> 11) * 2^-53."""
    u = (np_rng(seed, tag, idx) >> np.uint64(11)).astype(np.float64) * (2.0 ** -53)
    rank = np.searchsorted(cdf, u * cdf[-1], side="left")
    return np.minimum(rank, len(cdf) - 1).astype(np.uint64)


def np_rho(dist: str, seed: int, nR: int, nS: int, j: np.ndarray, z: float = 0.0, cdf=None) -> np.ndarray:
    j = j.astype(np.uint64)
    if dist == "fk":
        r = np_rng(seed, TAG_U, j) >> np.uint64(32)
        with np.errstate(over="ignore"):
            return (r * np.uint64(nR)) >> np.uint64(32)
    if dist == "1to1":
        assert nS == nR
        return np_perm_n(sub_seed(seed, TAG_S), nS, j)
    if dist == "zipf":
        if cdf is None:
            cdf = zipf_cdf(nR, z)
        u = (np_rng(seed, TAG_Z, j) >> np.uint64(11)).astype(np.float64) * (2.0 ** -53)
        t = u * cdf[-1]
        rank = np.searchsorted(cdf, t, side="left")
        rank = np.minimum(rank, nR - 1).astype(np.uint64)
        return np_perm_n(sub_seed(seed, TAG_Z), nR, rank)
    raise ValueError(dist)


# ----------------------------------------------------------------------------------------------
# torch implementation (int64 two's complement; wraps like uint64)
# ----------------------------------------------------------------------------------------------
def _to_i64(v: int) -> int:
    v &= M64
    return v - (1 << 64) if v >= (1 << 63) else v


def _srl(x, s: int):
    """Logical right shift of an int64 tensor holding uint64 bits."""
    import torch  # noqa: F401

    if s == 0:
        return x
    return (x >> s) & ((1 << (64 - s)) - 1)


def torch_fmix64(z):
    z = z ^ _srl(z, 30)
    z = z * _to_i64(0xBF58476D1CE4E5B9)
    z = z ^ _srl(z, 27)
    z = z * _to_i64(0x94D049BB133111EB)
    z = z ^ _srl(z, 31)
    return z


def torch_fmix32(h):
    m = 0xFFFFFFFF
    h = h & m
    h = h ^ (h >> 16)
    h = (h * 0x85EBCA6B) & m
    h = h ^ (h >> 13)
    h = (h * 0xC2B2AE35) & m
    h = h ^ (h >> 16)
    return h


def torch_rng(seed: int, tag: int, idx):
    base = _to_i64(fmix64_int(seed ^ tag))
    return torch_fmix64(idx * _to_i64(GOLDEN) + base)


def torch_perm_pow2(seed: int, k: int, x):
    import torch

    if k == 0:
        return torch.zeros_like(x)
    mask = (1 << k) - 1
    sh = (k + 1) // 2
    cs, as_ = perm_constants(seed)
    for r in range(4):
        x = (x + (cs[r] & mask)) & mask
        x = x ^ (x >> sh)
        x = (x * _to_i64(as_[r] & mask)) & mask
    return x


def torch_perm_n(seed: int, n: int, x):
    import torch

    k = _bits_for(n)
    y = torch_perm_pow2(seed, k, x)
    if n == (1 << k):
        return y
    bad = y >= n
    while bool(bad.any()):
        y = torch.where(bad, torch_perm_pow2(seed, k, y), y)
        bad = y >= n
    return y


def torch_keymap(kind: str, x, seed: int):
    import torch

    if kind == "dense":
        return x + 1
    if kind == "sparse":
        return torch_fmix32(x + 1)
    if kind == "k8":
        return torch_fmix64((x + 1) ^ _to_i64(sub_seed(seed, TAG_K)))
    raise ValueError(kind)


def torch_zrank(seed: int, tag: int, idx, cdf):
    import torch

    cdf_t = torch.from_numpy(cdf).to(idx.device)
    u = _srl(torch_rng(seed, tag, idx), 11).to(torch.float64) * (2.0 ** -53)
    return torch.searchsorted(cdf_t, u * cdf_t[-1], side="left").clamp_(max=len(cdf) - 1)


def torch_rho(dist: str, seed: int, nR: int, nS: int, j, z: float = 0.0, cdf=None):
    import torch

    if dist == "fk":
        r = _srl(torch_rng(seed, TAG_U, j), 32)
        return _srl(r * nR, 32) if nR < (1 << 32) else r
    if dist == "1to1":
        assert nS == nR
        return torch_perm_n(sub_seed(seed, TAG_S), nS, j)
    if dist == "zipf":
        if cdf is None:
            cdf = zipf_cdf(nR, z)
        cdf_t = torch.from_numpy(cdf).to(j.device)
        u = _srl(torch_rng(seed, TAG_Z, j), 11).to(torch.float64) * (2.0 ** -53)
        t = u * cdf_t[-1]
        rank = torch.searchsorted(cdf_t, t, side="left").clamp_(max=nR - 1)
        del t, u, cdf_t
        return torch_perm_n(sub_seed(seed, TAG_Z), nR, rank)
    raise ValueError(dist)


# ----------------------------------------------------------------------------------------------
# workload descriptions (BASELINE.json configs) and top-level generation
# ----------------------------------------------------------------------------------------------
@dataclasses.dataclass(frozen=True)
class Workload:
    name: str
    nR: int
    nS: int
    dist: str  # 'fk' | '1to1' | 'zipf'
    keys: str = "dense"  # 'dense' | 'sparse' | 'k8'
    z: float = 0.0
    seed: int = 1
    out_mode: int = 0  # 0 count+checksum, 1 materialize
    radix_bits: int = -1
    rep: int = 1  # 'replicas': copies of every key on each side

    @property
    def key_bytes(self) -> int:
        return 8 if self.keys == "k8" else 4

    @property
    def n(self) -> int:
        return self.nR + self.nS

    def with_(self, **kw) -> "Workload":
        return dataclasses.replace(self, **kw)


M = 1 << 20
CONFIGS = {
    # BASELINE.json configs[0..4]; seeds per SURVEY.md §8(c.3)
    "c1": Workload("c1", 1 * M, 1 * M, "fk", seed=1, out_mode=0, radix_bits=8),
    "c2": Workload("c2", 16 * M, 256 * M, "fk", seed=2, out_mode=0, radix_bits=12),
    "c3": Workload("c3", 128 * M, 128 * M, "1to1", seed=3, out_mode=1, radix_bits=15),
    "c4_z0.5": Workload("c4_z0.5", 16 * M, 256 * M, "zipf", z=0.5, seed=4, out_mode=0, radix_bits=12),
    "c4_z1.0": Workload("c4_z1.0", 16 * M, 256 * M, "zipf", z=1.0, seed=5, out_mode=0, radix_bits=12),
    "c4_z1.5": Workload("c4_z1.5", 16 * M, 256 * M, "zipf", z=1.5, seed=6, out_mode=0, radix_bits=12),
    "c5": Workload("c5", 2048 * M, 2048 * M, "1to1", keys="k8", seed=7, out_mode=0, radix_bits=19),
    # one GPU's share of c5 at 8 GPUs (2^28 x 2^28, 8 B keys / payloads), for single-GPU runs
    "c5_gpu": Workload("c5_gpu", 256 * M, 256 * M, "1to1", keys="k8", seed=7, out_mode=0, radix_bits=16),
}


SKEW_DISTS = ("zipf_build", "zipf_both", "replicas")


def np_generate(w: Workload, s_rows: slice | None = None, cdf=None):
    """Return (R_key, R_pay, S_key, S_pay) as numpy arrays (host).

    ``s_rows`` restricts S to a row range (the counter-based generator makes
    any row range independently computable)."""
    pay_dt = np.uint64 if w.keys == "k8" else np.uint32
    i = np.arange(w.nR, dtype=np.uint64)
    lo, hi = (0, w.nS) if s_rows is None else (s_rows.start, s_rows.stop)
    j = np.arange(lo, hi, dtype=np.uint64)
    if w.dist in SKEW_DISTS:
        xR, xS = np_skew_x(w, i, j)
        return (np_keymap(w.keys, xR, w.seed), i.astype(pay_dt), np_keymap(w.keys, xS, w.seed), j.astype(pay_dt))
    xR = np_perm_n(sub_seed(w.seed, TAG_R), w.nR, i)
    Rk = np_keymap(w.keys, xR, w.seed)
    Rp = i.astype(pay_dt)
    del xR
    rho = np_rho(w.dist, w.seed, w.nR, w.nS, j, w.z, cdf)
    Sk = Rk[rho.astype(np.int64)]
    Sp = j.astype(pay_dt)
    return Rk, Rp, Sk, Sp


def np_skew_x(w: Workload, i: np.ndarray, j: np.ndarray):
    """Domain indices of the NEXT-2 workloads (see the module docstring)."""
    if w.dist == "zipf_build":
        cdf = zipf_cdf(w.nS, w.z)
        xR = np_perm_n(sub_seed(w.seed, TAG_Z), w.nS, np_zrank(w.seed, TAG_B, i, cdf))
        xS = np_perm_n(sub_seed(w.seed, TAG_S), w.nS, j)
    elif w.dist == "zipf_both":
        cdf = zipf_cdf(w.nR, w.z)
        xR = np_perm_n(sub_seed(w.seed, TAG_Z), w.nR, np_zrank(w.seed, TAG_B, i, cdf))
        xS = np_perm_n(sub_seed(w.seed, TAG_Z), w.nR, np_zrank(w.seed, TAG_Z, j, cdf))
    else:  # replicas
        D = np.uint64(max(1, w.nR // w.rep))
        xR = np_perm_n(sub_seed(w.seed, TAG_R), w.nR, i) % D
        xS = np_perm_n(sub_seed(w.seed, TAG_S), w.nS, j) % D
    return xR, xS


def np_rho_for(w: Workload, j: np.ndarray, cdf=None) -> np.ndarray:
    return np_rho(w.dist, w.seed, w.nR, w.nS, j, w.z, cdf)


def torch_generate(w: Workload, device="cuda", cdf=None):
    """Same columns as np_generate, created directly on ``device``.

    4-byte columns come back as torch.int32 tensors holding the uint32 bits;
    8-byte columns as torch.int64 holding the uint64 bits."""
    import torch

    i = torch.arange(w.nR, dtype=torch.int64, device=device)
    j = torch.arange(w.nS, dtype=torch.int64, device=device)
    if w.dist in SKEW_DISTS:
        if w.dist == "zipf_build":
            c = zipf_cdf(w.nS, w.z)
            xR = torch_perm_n(sub_seed(w.seed, TAG_Z), w.nS, torch_zrank(w.seed, TAG_B, i, c))
            xS = torch_perm_n(sub_seed(w.seed, TAG_S), w.nS, j)
        elif w.dist == "zipf_both":
            c = zipf_cdf(w.nR, w.z)
            xR = torch_perm_n(sub_seed(w.seed, TAG_Z), w.nR, torch_zrank(w.seed, TAG_B, i, c))
            xS = torch_perm_n(sub_seed(w.seed, TAG_Z), w.nR, torch_zrank(w.seed, TAG_Z, j, c))
        else:
            D = max(1, w.nR // w.rep)
            xR = torch_perm_n(sub_seed(w.seed, TAG_R), w.nR, i) % D
            xS = torch_perm_n(sub_seed(w.seed, TAG_S), w.nS, j) % D
        Rk64, Sk64 = torch_keymap(w.keys, xR, w.seed), torch_keymap(w.keys, xS, w.seed)
        del xR, xS
    else:
        xR = torch_perm_n(sub_seed(w.seed, TAG_R), w.nR, i)
        Rk64 = torch_keymap(w.keys, xR, w.seed)
        del xR
        rho = torch_rho(w.dist, w.seed, w.nR, w.nS, j, w.z, cdf)
        Sk64 = Rk64[rho]
        del rho
    if w.keys == "k8":
        return Rk64, i, Sk64, j
    return (_as_u32_bits(Rk64), _as_u32_bits(i), _as_u32_bits(Sk64), _as_u32_bits(j))


def _as_u32_bits(t):
    """int64 tensor holding values in [0, 2^32) -> int32 tensor with the same low 32 bits."""
    import torch

    t = t & 0xFFFFFFFF
    return torch.where(t >= (1 << 31), t - (1 << 32), t).to(torch.int32)


def expected_matches_closed_form(w: Workload) -> int | None:
    """FK and 1:1 joins over unique R keys produce exactly one match per S row (every S key is
    some R key and R keys are unique); a build-skewed R over a domain S covers exactly once
    produces one match per R row; replicas produce rep matches per R row when rep | nR, nS."""
    if w.dist in ("fk", "1to1", "zipf"):
        return w.nS
    if w.dist == "zipf_build":
        return w.nR
    if w.dist == "replicas" and w.nR % w.rep == 0 and w.nS % (w.nR // w.rep) == 0:
        return w.nR * (w.nS // (w.nR // w.rep))
    return None
