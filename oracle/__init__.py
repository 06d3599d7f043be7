"""CPU oracle for the radix-partitioned hash join -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline`` /
``--impl reference`` legs may import this package. The product package
(``paper_conf_icde_sioulasckaa19_b200``) never imports it and shares no code with it.

Thin ctypes wrapper over ``hj_oracle.c`` (plain single-threaded C; see its header for
the result definition and the passages of PAPER.md each function follows).

Parity pins (tests/test_oracle.py): brute-force nested loop, numpy sort-merge count,
generator closed forms, a hand-worked golden example, and published splitmix64 outputs.
Every oracle function is pinned; none is "parity unpinned".
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "hj_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lib = None


def build(force: bool = False) -> str:
    """Compile hj_oracle.c with plain gcc -O2 (no OpenMP, no vectorization flags)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-shared", "-fPIC", "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        u64, i32, vp = ctypes.c_uint64, ctypes.c_int, ctypes.c_void_p
        lib.oracle_hash_join.argtypes = [i32, i32, vp, vp, u64, vp, vp, u64, i32, u64, vp, vp, u64,
                                         ctypes.POINTER(u64), ctypes.POINTER(u64)]
        lib.oracle_hash_join.restype = i32
        lib.oracle_radix_partition.argtypes = [i32, i32, vp, vp, u64, i32, i32, vp, vp, vp]
        lib.oracle_radix_partition.restype = i32
        lib.oracle_sig.argtypes = [u64, u64]
        lib.oracle_sig.restype = u64
        lib.oracle_fmix64.argtypes = [u64]
        lib.oracle_fmix64.restype = u64
        _lib = lib
    return _lib


def _col(a: np.ndarray, width: int) -> np.ndarray:
    dt = np.uint32 if width == 4 else np.uint64
    a = np.ascontiguousarray(a)
    if a.dtype != dt:
        if a.dtype.itemsize != width:
            raise ValueError(f"column has {a.dtype.itemsize}-byte elements, expected {width}")
        a = a.view(dt)
    return a


def _ptr(a: np.ndarray):
    return a.ctypes.data_as(ctypes.c_void_p) if a.size else None


def sig(r_pay: int, s_pay: int) -> int:
    return int(_load().oracle_sig(r_pay, s_pay))


def fmix64(z: int) -> int:
    return int(_load().oracle_fmix64(z))


def hash_join(R_keys, R_pay, S_keys, S_pay, materialize: bool = False, slice_bits: int = 0,
              slice_id: int = 0, cap: int | None = None):
    """Canonical hash join R ⋈ S.

    Returns (matches, checksum) or, with ``materialize``, (matches, checksum, r_pay_out, s_pay_out)
    with pairs in probe order (compare after a lexicographic sort)."""
    kb = R_keys.dtype.itemsize
    pb = R_pay.dtype.itemsize
    Rk, Rp, Sk, Sp = _col(R_keys, kb), _col(R_pay, pb), _col(S_keys, kb), _col(S_pay, pb)
    nR, nS = len(Rk), len(Sk)
    assert len(Rp) == nR and len(Sp) == nS
    m, c = ctypes.c_uint64(0), ctypes.c_uint64(0)
    if materialize:
        if cap is None:
            # the result size is unknown: count first, then materialize exactly
            rc = _load().oracle_hash_join(kb, pb, _ptr(Rk), _ptr(Rp), nR, _ptr(Sk), _ptr(Sp), nS,
                                          slice_bits, slice_id, None, None, 0, ctypes.byref(m), ctypes.byref(c))
            if rc != 0:
                raise RuntimeError(f"oracle_hash_join failed: {rc}")
            cap = int(m.value)
        dt = np.uint32 if pb == 4 else np.uint64
        out_r = np.zeros(cap, dtype=dt)
        out_s = np.zeros(cap, dtype=dt)
        rc = _load().oracle_hash_join(kb, pb, _ptr(Rk), _ptr(Rp), nR, _ptr(Sk), _ptr(Sp), nS, slice_bits,
                                      slice_id, _ptr(out_r), _ptr(out_s), cap, ctypes.byref(m), ctypes.byref(c))
        if rc != 0:
            raise RuntimeError(f"oracle_hash_join failed: {rc}")
        k = min(cap, int(m.value))
        return int(m.value), int(c.value), out_r[:k], out_s[:k]
    rc = _load().oracle_hash_join(kb, pb, _ptr(Rk), _ptr(Rp), nR, _ptr(Sk), _ptr(Sp), nS, slice_bits, slice_id,
                                  None, None, 0, ctypes.byref(m), ctypes.byref(c))
    if rc != 0:
        raise RuntimeError(f"oracle_hash_join failed: {rc}")
    return int(m.value), int(c.value)


def radix_partition(keys, pays, shift: int, bits: int):
    """Stable counting sort by digit (key >> shift) & (2^bits-1) (Fig. 1).

    Returns (out_keys, out_pays, offsets[2^bits + 1])."""
    kb, pb = keys.dtype.itemsize, pays.dtype.itemsize
    k, p = _col(keys, kb), _col(pays, pb)
    ok = np.empty_like(k)
    op = np.empty_like(p)
    offs = np.zeros((1 << bits) + 1, dtype=np.uint64)
    rc = _load().oracle_radix_partition(kb, pb, _ptr(k), _ptr(p), len(k), shift, bits, _ptr(ok), _ptr(op),
                                        offs.ctypes.data_as(ctypes.c_void_p))
    if rc != 0:
        raise RuntimeError(f"oracle_radix_partition failed: {rc}")
    return ok, op, offs


def pairs_sorted(r, s) -> np.ndarray:
    """Pairs as a (m, 2) uint64 array sorted lexicographically (reading S9)."""
    r = np.asarray(r).astype(np.uint64)
    s = np.asarray(s).astype(np.uint64)
    order = np.lexsort((s, r))
    return np.stack([r[order], s[order]], axis=1)
