"""B200-native radix-partitioned hash join (Sioulas et al., ICDE 2019) -- Python binding.

Argument marshalling only: every step of the join runs in the sm_100a kernels of
``libhj.so`` behind the C-ABI of ``include/hj.h``. There is no CPU fallback: importing
this package without the built library raises, and so does calling it without a CUDA
device. PyTorch supplies device memory and streams.

    import paper_conf_icde_sioulasckaa19_b200 as hj
    res = hj.join(R_keys, R_pay, S_keys, S_pay, radix_bits=-1, out_mode=hj.OUT_COUNT_CHECKSUM)
    res.matches, res.checksum                      # python ints (uint64 semantics)
    res = hj.join(..., out_mode=hj.OUT_MATERIALIZE)
    res.r_pay, res.s_pay                           # torch CUDA tensors of `matches` payloads

Columns are 1-D contiguous CUDA tensors of 4-byte (int32/uint32 bits) or 8-byte
(int64/uint64 bits) elements; key and payload widths must match (4/4 or 8/8).
"""
from __future__ import annotations

import ctypes
import dataclasses
import os
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("HJ_LIB") or os.path.join(_HERE, "libhj.so")  # HJ_LIB: an experimental build

OUT_COUNT_CHECKSUM = 0
OUT_MATERIALIZE = 1

OPT_CAP_R = 1
OPT_CHUNK_S = 2
OPT_OUT_CAPACITY = 3
OPT_TIMING = 4
OPT_BLOCKS_PER_SM = 5
OPT_JOIN_VARIANT = 6
OPT_PASS_THREADS = 7
OPT_STREAM_CHUNK = 8
OPT_JOIN_ALGO = 9
OPT_GRAPH = 11
OPT_PARTITIONER = 12  # 0 = histogram (default), 1 = bucket chains (NEXT-1)
OPT_PASS_L2PF = 17
OPT_PASS1_BITS = 18
OPT_PASS_VARIANT = 19
OPT_MAT_CHECKSUM = 20  # 1 (default): MATERIALIZE also returns the checksum
OPT_PASS_WS = 21  # 1 (default): warp-specialized partition passes
OPT_PDL = 22  # 1: programmatic dependent launch between the kernels of a call
ALGO_HASH, ALGO_NLJ, ALGO_NONPARTITIONED = 0, 1, 2

ERR_WORKSPACE = -6
_ERRORS = {-1: "HJ_ERR_INVALID", -2: "HJ_ERR_UNSUPPORTED", -3: "HJ_ERR_OOM", -4: "HJ_ERR_CUDA", -5: "HJ_ERR_COMM",
           -6: "HJ_ERR_WORKSPACE"}

# every symbol include/hj.h declares (checked by tests/test_abi.py)
EXPORTS = ("hj_create", "hj_destroy", "hj_last_error", "hj_set_stream", "hj_set_option", "hj_join",
           "hj_join_async", "hj_sync",
           "hj_workspace_bytes", "hj_set_workspace", "hj_join_host", "hj_partition", "hj_exchange_pack",
           "hj_exchange_row_len", "hj_join_received", "hj_xd_window",
           "hj_xd_header_bytes", "hj_ipc_open", "hj_ipc_close", "hj_xd_count", "hj_xd_store", "hj_xd_barrier",
           "hj_xd_join", "hj_xd_reserve", "hj_version")
XD_MAX_RANKS = 64
MAX_PENDING = 8         # HJ_MAX_PENDING
XD_BOARD_BYTES = 69632  # HJ_XD_BOARD_BYTES
XD_REGROW = 1           # HJ_XD_REGROW


class HJError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"{_ERRORS.get(code, code)}: {msg}")
        self.code = code


class _Result(ctypes.Structure):
    _fields_ = [("matches", ctypes.c_uint64), ("checksum", ctypes.c_uint64), ("r_pay_out", ctypes.c_void_p),
                ("s_pay_out", ctypes.c_void_p), ("n_items", ctypes.c_uint64), ("radix_bits", ctypes.c_int),
                ("passes", ctypes.c_int), ("ms_total", ctypes.c_float), ("ms_partition", ctypes.c_float),
                ("ms_join", ctypes.c_float), ("ms_kernel", ctypes.c_float * 5), ("kernels", ctypes.c_uint32),
                ("reserved", ctypes.c_uint32)]


def _load_lib():
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"{LIB_PATH} is missing: build it with `make` or __graft_entry__.build() "
                          "(there is no CPU fallback)")
    lib = ctypes.CDLL(LIB_PATH)
    vp, u64, i32, i64 = ctypes.c_void_p, ctypes.c_uint64, ctypes.c_int, ctypes.c_int64
    lib.hj_create.argtypes = [ctypes.POINTER(vp), i32, i32, i32, vp]
    lib.hj_create.restype = i32
    lib.hj_destroy.argtypes = [vp]
    lib.hj_destroy.restype = None
    lib.hj_last_error.argtypes = [vp]
    lib.hj_last_error.restype = ctypes.c_char_p
    lib.hj_set_stream.argtypes = [vp, vp]
    lib.hj_set_stream.restype = i32
    lib.hj_set_option.argtypes = [vp, i32, i64]
    lib.hj_set_option.restype = i32
    for f in (lib.hj_join, lib.hj_join_host, lib.hj_join_async):
        f.argtypes = [vp, vp, vp, u64, vp, vp, u64, i32, i32, ctypes.POINTER(_Result)]
        f.restype = i32
    lib.hj_sync.argtypes = [vp]
    lib.hj_sync.restype = i32
    lib.hj_workspace_bytes.argtypes = [vp, u64, u64, i32, i32]
    lib.hj_workspace_bytes.restype = u64
    lib.hj_set_workspace.argtypes = [vp, vp, u64]
    lib.hj_set_workspace.restype = i32
    lib.hj_partition.argtypes = [vp, vp, vp, u64, i32, ctypes.POINTER(vp), ctypes.POINTER(u64), ctypes.POINTER(u64)]
    lib.hj_partition.restype = i32
    lib.hj_exchange_pack.argtypes = [vp, i32, vp, vp, u64, i32, i32, ctypes.POINTER(vp), ctypes.POINTER(vp),
                                     ctypes.POINTER(u64)]
    lib.hj_exchange_pack.restype = i32
    lib.hj_join_received.argtypes = [vp, vp, u64, vp, vp, u64, vp, i32, i32, i32, ctypes.POINTER(_Result)]
    lib.hj_join_received.restype = i32
    lib.hj_xd_window.argtypes = [vp, i32, u64, ctypes.POINTER(vp), vp, ctypes.POINTER(i32)]
    lib.hj_xd_window.restype = i32
    lib.hj_xd_header_bytes.argtypes = [i32, i32]
    lib.hj_xd_header_bytes.restype = u64
    lib.hj_exchange_row_len.argtypes = [i32, i32]
    lib.hj_exchange_row_len.restype = ctypes.c_uint32
    lib.hj_ipc_open.argtypes = [vp, vp, ctypes.POINTER(vp)]
    lib.hj_ipc_open.restype = i32
    lib.hj_ipc_close.argtypes = [vp, vp]
    lib.hj_ipc_close.restype = i32
    lib.hj_xd_count.argtypes = [vp, vp, vp, u64, vp, vp, u64, i32, i32, ctypes.POINTER(u64)]
    lib.hj_xd_count.restype = i32
    lib.hj_xd_store.argtypes = [vp, i32, ctypes.POINTER(u64), ctypes.POINTER(vp), ctypes.POINTER(vp)]
    lib.hj_xd_store.restype = i32
    lib.hj_xd_barrier.argtypes = [vp, i32, i32, ctypes.POINTER(vp), ctypes.c_uint32]
    lib.hj_xd_barrier.restype = i32
    lib.hj_xd_join.argtypes = [vp, i32, i32, vp, vp, u64, vp, vp, u64, i32, i32, ctypes.POINTER(vp),
                               ctypes.POINTER(vp), ctypes.POINTER(vp), ctypes.POINTER(u64), ctypes.c_uint32,
                               ctypes.POINTER(_Result), ctypes.POINTER(u64), ctypes.POINTER(u64)]
    lib.hj_xd_join.restype = i32
    lib.hj_xd_reserve.argtypes = [vp, i32, u64, u64, i32, i32, u64, u64]
    lib.hj_xd_reserve.restype = i32
    lib.hj_version.argtypes = []
    lib.hj_version.restype = ctypes.c_char_p
    return lib


_lib = _load_lib()


def lib():
    return _lib


def version() -> str:
    return _lib.hj_version().decode()


@dataclasses.dataclass
class JoinResult:
    matches: int
    checksum: int
    r_pay: object = None  # torch tensor (device) or numpy array (host) when materialized
    s_pay: object = None
    n_items: int = 0
    radix_bits: int = 0
    passes: int = 0
    ms_total: float = 0.0
    ms_partition: float = 0.0
    ms_join: float = 0.0
    ms_kernel: tuple = ()
    kernels: int = 0


class Context:
    """One hj_ctx (device, widths). Not thread-safe; the module keeps one per thread.

    With workspace=True (default) hj_join's device memory is a torch tensor this object owns
    (hj_workspace_bytes / hj_set_workspace): PyTorch's caching allocator supplies it, and the
    library neither allocates nor synchronizes inside hj_join before the result readback."""

    def __init__(self, device: int = 0, key_bytes: int = 4, pay_bytes: int = 4, stream: int | None = None,
                 workspace: bool = True):
        h = ctypes.c_void_p()
        rc = _lib.hj_create(ctypes.byref(h), device, key_bytes, pay_bytes, stream)
        if rc != 0:
            raise HJError(rc, _lib.hj_last_error(None).decode())
        self._h = h
        self.device = device
        self.key_bytes = key_bytes
        self.pay_bytes = pay_bytes
        self.use_workspace = workspace
        self._ws = None  # torch uint8 tensor backing hj_join's buffers
        self._pending = []  # join_async calls not yet returned by sync(): (result struct, columns, mode, device)

    def close(self):
        self._view_key = self._view_val = None  # views of memory hj_destroy frees
        if getattr(self, "_h", None):
            _lib.hj_destroy(self._h)  # completes pending join_async calls first
            self._h = None
        self._pending = []
        self._ws = None  # after hj_destroy: the ctx no longer touches it

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def _check(self, rc):
        if rc != 0:
            raise HJError(rc, _lib.hj_last_error(self._h).decode())

    def set_option(self, opt: int, value: int):
        self._check(_lib.hj_set_option(self._h, opt, int(value)))

    def set_stream(self, stream_handle: int | None):
        self._check(_lib.hj_set_stream(self._h, stream_handle))

    def workspace_bytes(self, nR: int, nS: int, radix_bits: int = -1, out_mode: int = OUT_COUNT_CHECKSUM) -> int:
        return int(_lib.hj_workspace_bytes(self._h, nR, nS, radix_bits, out_mode))

    def _ensure_workspace(self, nbytes: int, device):
        import torch

        if self._ws is not None and self._ws.numel() >= nbytes:
            return
        self._view_key = self._view_val = None
        self._check(_lib.hj_set_workspace(self._h, None, 0))  # drop the old one before torch frees it
        self._ws = None
        # +256: torch's allocations are 512-byte aligned already; the slack keeps the size a multiple
        self._ws = torch.empty(nbytes + 256, dtype=torch.uint8, device=device)
        self._check(_lib.hj_set_workspace(self._h, ctypes.c_void_p(self._ws.data_ptr()), self._ws.numel()))

    def join(self, Rk, Rp, Sk, Sp, radix_bits: int = -1, out_mode: int = OUT_COUNT_CHECKSUM) -> JoinResult:
        import torch

        cols = [_as_device_col(t, self.key_bytes if i % 2 == 0 else self.pay_bytes) for i, t in enumerate((Rk, Rp, Sk, Sp))]
        if cols[0].numel() != cols[1].numel() or cols[2].numel() != cols[3].numel():
            raise ValueError("key and payload columns differ in length")
        dev_ = cols[0].device
        self.set_stream(torch.cuda.current_stream(dev_).cuda_stream)
        nR, nS = cols[0].numel(), cols[2].numel()
        res = _Result()
        for _ in range(3):
            if self.use_workspace and nR and nS:
                self._ensure_workspace(self.workspace_bytes(nR, nS, radix_bits, out_mode), dev_)
            rc = _lib.hj_join(self._h, _ptr(cols[0]), _ptr(cols[1]), nR, _ptr(cols[2]), _ptr(cols[3]), nS,
                              radix_bits, out_mode, ctypes.byref(res))
            if rc != ERR_WORKSPACE or not self.use_workspace:
                break
            # materialized pairs outgrew the capacity (reading S11: never overwrite): the exact
            # count came back in res.matches -> grow the output part of the workspace, re-run
            self.set_option(OPT_OUT_CAPACITY, max(int(res.matches), 1))
        self._check(rc)
        out = _result(res)
        if out_mode == OUT_MATERIALIZE and res.matches:
            out.r_pay, out.s_pay = self._views(res, dev_)
        return out

    def join_async(self, Rk, Rp, Sk, Sp, radix_bits: int = -1, out_mode: int = OUT_COUNT_CHECKSUM) -> int:
        """hj_join_async: enqueue the join on torch's current stream and return at once; sync()
        returns the results of every pending call in issue order. The columns are kept alive
        until then. Returns the call's index in the next sync() list."""
        import torch

        cols = [_as_device_col(t, self.key_bytes if i % 2 == 0 else self.pay_bytes) for i, t in enumerate((Rk, Rp, Sk, Sp))]
        if cols[0].numel() != cols[1].numel() or cols[2].numel() != cols[3].numel():
            raise ValueError("key and payload columns differ in length")
        dev_ = cols[0].device
        self.set_stream(torch.cuda.current_stream(dev_).cuda_stream)
        nR, nS = cols[0].numel(), cols[2].numel()
        if self.use_workspace and nR and nS:
            self._ensure_workspace(self.workspace_bytes(nR, nS, radix_bits, out_mode), dev_)
        res = _Result()
        self._check(_lib.hj_join_async(self._h, _ptr(cols[0]), _ptr(cols[1]), nR, _ptr(cols[2]), _ptr(cols[3]), nS,
                                       radix_bits, out_mode, ctypes.byref(res)))
        self._pending.append((res, cols, out_mode, dev_))
        return len(self._pending) - 1

    def sync(self) -> list:
        """hj_sync: wait for every pending join_async call; their JoinResults in issue order.
        MATERIALIZE: the pending calls share the output buffer, so only the last result carries
        the pair views (the last call's pairs)."""
        pend, self._pending = self._pending, []
        self._check(_lib.hj_sync(self._h))
        out = [_result(r) for r, _, _, _ in pend]
        if pend and pend[-1][2] == OUT_MATERIALIZE and pend[-1][0].matches:
            out[-1].r_pay, out[-1].s_pay = self._views(pend[-1][0], pend[-1][3])
        return out

    def _views(self, res, device):
        # the ctx-owned output buffers are stable across calls (until regrown): the torch views
        # are built once per (pointers, count) instead of per call (host overhead between calls)
        key = (res.r_pay_out, res.s_pay_out, res.matches, device)
        if getattr(self, "_view_key", None) != key:
            self._view_val = (_wrap_device(res.r_pay_out, res.matches, self.pay_bytes, device),
                              _wrap_device(res.s_pay_out, res.matches, self.pay_bytes, device))
            self._view_key = key
        return self._view_val

    def join_host(self, Rk, Rp, Sk, Sp, radix_bits: int = -1, out_mode: int = OUT_COUNT_CHECKSUM,
                  copy: bool = True) -> JoinResult:
        """End-to-end call from host numpy columns (H2D copies, join, D2H of the result).
        With copy=False the materialized pairs are numpy views of the ctx's pinned buffer,
        valid until the next call on this context."""
        cols = [np.ascontiguousarray(a) for a in (Rk, Rp, Sk, Sp)]
        for i, a in enumerate(cols):
            want = self.key_bytes if i % 2 == 0 else self.pay_bytes
            if a.dtype.itemsize != want:
                raise ValueError(f"column {i} has {a.dtype.itemsize}-byte elements, expected {want}")
        self.set_stream(None)
        res = _Result()
        rc = _lib.hj_join_host(self._h, _nptr(cols[0]), _nptr(cols[1]), len(cols[0]), _nptr(cols[2]), _nptr(cols[3]),
                               len(cols[2]), radix_bits, out_mode, ctypes.byref(res))
        self._check(rc)
        out = _result(res)
        if out_mode == OUT_MATERIALIZE and res.matches:
            dt = np.uint32 if self.pay_bytes == 4 else np.uint64
            n = res.matches
            buf_r = (ctypes.c_char * (n * self.pay_bytes)).from_address(res.r_pay_out)
            buf_s = (ctypes.c_char * (n * self.pay_bytes)).from_address(res.s_pay_out)
            out.r_pay = np.frombuffer(buf_r, dtype=dt)
            out.s_pay = np.frombuffer(buf_s, dtype=dt)
            if copy:
                out.r_pay, out.s_pay = out.r_pay.copy(), out.s_pay.copy()
        return out

    def partition(self, keys, pays, radix_bits: int):
        """Steps a1-a4 on one relation. Returns (tuples, part_start, part_count): tuples is a
        torch tensor view of the ctx-owned AoS buffer (int64 per 4/4 tuple, or [n, 2] int64 for
        8/8), valid until the next call on this context."""
        import torch

        k = _as_device_col(keys, self.key_bytes)
        p = _as_device_col(pays, self.pay_bytes)
        self.set_stream(torch.cuda.current_stream(k.device).cuda_stream)
        np_ = 1 << radix_bits
        start = (ctypes.c_uint64 * np_)()
        count = (ctypes.c_uint64 * np_)()
        out = ctypes.c_void_p()
        self._check(_lib.hj_partition(self._h, _ptr(k), _ptr(p), k.numel(), radix_bits, ctypes.byref(out), start, count))
        n = k.numel()
        tw = self.key_bytes + self.pay_bytes
        t = _wrap_device(out.value, n * tw // 8, 8, k.device) if n else torch.zeros(0, dtype=torch.int64, device=k.device)
        if self.key_bytes == 8:
            t = t.view(n, 2)
        return t, np.frombuffer(start, dtype=np.uint64).copy(), np.frombuffer(count, dtype=np.uint64).copy()


    # ---- multi-GPU exchange (used by paper_conf_icde_sioulasckaa19_b200.dist) -------------------
    def exchange_pack(self, rel: int, keys, pays, gpu_bits: int, local_bits: int):
        """Rows a1-a3 with the pass-1 digit widened by `gpu_bits` rank bits (hj_exchange_pack).
        Returns (send, counts, dest): send = int64 tensor view of the AoS send buffer (one word per
        4/4 tuple, two per 8/8 tuple), counts = int32 tensor [G, row_len] of piece counts (row j
        goes to rank j: its tuples per pass-1 digit d1, row_len = exchange_row_len(G, local_bits)),
        dest = numpy uint64 [G] tuples per destination. Views are ctx-owned (valid until the next
        pack of the same relation)."""
        import torch

        k = _as_device_col(keys, self.key_bytes)
        p = _as_device_col(pays, self.pay_bytes)
        self.set_stream(torch.cuda.current_stream(k.device).cuda_stream)
        G = 1 << gpu_bits
        send, cnt = ctypes.c_void_p(), ctypes.c_void_p()
        dest = (ctypes.c_uint64 * G)()
        self._check(_lib.hj_exchange_pack(self._h, rel, _ptr(k), _ptr(p), k.numel(), gpu_bits, local_bits,
                                          ctypes.byref(send), ctypes.byref(cnt), dest))
        words = k.numel() * (self.key_bytes + self.pay_bytes) // 8
        send_t = (_wrap_device(send.value, words, 8, k.device) if words
                  else torch.zeros(0, dtype=torch.int64, device=k.device))
        rl = exchange_row_len(G, local_bits)
        cnt_t = _wrap_device(cnt.value, G * rl, 4, k.device).view(G, rl)
        return send_t, cnt_t, np.frombuffer(dest, dtype=np.uint64).copy()

    def join_received(self, R_recv, nR: int, R_counts, S_recv, nS: int, S_counts, nsrc: int, local_bits: int,
                      out_mode: int = OUT_COUNT_CHECKSUM) -> JoinResult:
        """Rows a4-a8 on received tuples (hj_join_received): this rank's share of the join."""
        import torch

        dev_ = R_counts.device
        self.set_stream(torch.cuda.current_stream(dev_).cuda_stream)
        for t in (R_recv, S_recv, R_counts, S_counts):
            if not t.is_cuda or not t.is_contiguous():
                raise ValueError("join_received takes contiguous CUDA tensors")
        res = _Result()
        self._check(_lib.hj_join_received(self._h, _ptr(R_recv), nR, _ptr(R_counts), _ptr(S_recv), nS,
                                          _ptr(S_counts), nsrc, local_bits, out_mode, ctypes.byref(res)))
        out = _result(res)
        if out_mode == OUT_MATERIALIZE and res.matches:
            out.r_pay = _wrap_device(res.r_pay_out, res.matches, self.pay_bytes, dev_)
            out.s_pay = _wrap_device(res.s_pay_out, res.matches, self.pay_bytes, dev_)
        return out


    # ---- direct-store exchange (hj_xd_*; orchestrated by dist.DirectExchange) -----------------
    def xd_window(self, slot: int, nbytes: int, want_handle: bool = True):
        """(re)allocate window `slot` (0 R, 1 S, 2 flags) to >= nbytes -> (dptr, handle bytes | None, grew)."""
        d = ctypes.c_void_p()
        grew = ctypes.c_int()
        hb = ctypes.create_string_buffer(64) if want_handle else None
        self._check(_lib.hj_xd_window(self._h, slot, int(nbytes), ctypes.byref(d), hb, ctypes.byref(grew)))
        return int(d.value), (hb.raw if hb is not None else None), bool(grew.value)

    def ipc_open(self, handle: bytes) -> int:
        d = ctypes.c_void_p()
        self._check(_lib.hj_ipc_open(self._h, ctypes.create_string_buffer(handle, 64), ctypes.byref(d)))
        return int(d.value)

    def ipc_close(self, dptr: int):
        self._check(_lib.hj_ipc_close(self._h, ctypes.c_void_p(dptr)))

    def xd_count(self, Rk, Rp, Sk, Sp, gpu_bits: int, local_bits: int):
        """Rows a1-a2 (hj_xd_count) -> numpy uint64 [2, G]: tuples of R / S sent to each rank."""
        import torch

        cols = [_as_device_col(Rk, self.key_bytes), _as_device_col(Rp, self.pay_bytes),
                _as_device_col(Sk, self.key_bytes), _as_device_col(Sp, self.pay_bytes)]
        self.set_stream(torch.cuda.current_stream(cols[0].device).cuda_stream)
        G = 1 << gpu_bits
        dest = (ctypes.c_uint64 * (2 * G))()
        self._check(_lib.hj_xd_count(self._h, _ptr(cols[0]), _ptr(cols[1]), cols[0].numel(), _ptr(cols[2]),
                                     _ptr(cols[3]), cols[2].numel(), gpu_bits, local_bits, dest))
        return np.frombuffer(dest, dtype=np.uint64).reshape(2, G).copy()

    def xd_store(self, rank: int, totals, win_R, win_S):
        """Row a3 into the peers' windows (hj_xd_store). totals: uint64 [2, G, G]; win_*: G device addresses."""
        t = np.ascontiguousarray(totals, dtype=np.uint64)
        G = t.shape[1]
        wr = (ctypes.c_void_p * G)(*[int(x) for x in win_R])
        ws = (ctypes.c_void_p * G)(*[int(x) for x in win_S])
        self._check(_lib.hj_xd_store(self._h, rank, t.ctypes.data_as(ctypes.POINTER(ctypes.c_uint64)), wr, ws))

    def xd_header_bytes(self, G: int, local_bits: int) -> int:
        return xd_header_bytes(G, local_bits)

    def xd_views(self, dptr: int, G: int, local_bits: int, n: int, device):
        """Torch views of a receive window: (tuples as int64 words, piece-count rows int32 [G, row_len])."""
        H = xd_header_bytes(G, local_bits)
        words = n * (self.key_bytes + self.pay_bytes) // 8
        recv = _wrap_device(dptr + H, max(words, 1), 8, device)[:words]
        rl = exchange_row_len(G, local_bits)
        cnt = _wrap_device(dptr, G * rl, 4, device).view(G, rl)
        return recv, cnt

    def xd_barrier(self, rank: int, flags, timeout_ms: int = 10000):
        G = len(flags)
        f = (ctypes.c_void_p * G)(*[int(x) for x in flags])
        self._check(_lib.hj_xd_barrier(self._h, rank, G, f, timeout_ms))


    def xd_join(self, rank: int, gpu_bits: int, Rk, Rp, Sk, Sp, local_bits: int, out_mode: int, win_R, win_S,
                board, win_bytes, timeout_ms: int = 10000):
        """The device-driven multi-GPU join of this rank (hj_xd_join).
        Returns (status, JoinResult of this rank's share, totals uint64 [2, G, G], (matches, checksum)
        over all ranks); status XD_REGROW = windows too small, nothing joined (grow and call again)."""
        import torch

        cols = [_as_device_col(Rk, self.key_bytes), _as_device_col(Rp, self.pay_bytes),
                _as_device_col(Sk, self.key_bytes), _as_device_col(Sp, self.pay_bytes)]
        dev_ = cols[0].device
        self.set_stream(torch.cuda.current_stream(dev_).cuda_stream)
        G = 1 << gpu_bits
        # the marshalled window tables are rebuilt only when the windows change (per-call host
        # time is on the multi-GPU critical path)
        cap = np.ascontiguousarray(win_bytes, dtype=np.uint64).reshape(2, G)
        key = (tuple(int(x) for x in win_R), tuple(int(x) for x in win_S), tuple(int(x) for x in board), cap.tobytes())
        xc = getattr(self, "_xd_marshal", None)
        if xc is None or xc[0] != key:
            u64p = ctypes.POINTER(ctypes.c_uint64)
            tot, allv = np.zeros((2, G, G), dtype=np.uint64), np.zeros(2, dtype=np.uint64)
            xc = self._xd_marshal = (key, (ctypes.c_void_p * G)(*key[0]), (ctypes.c_void_p * G)(*key[1]),
                                     (ctypes.c_void_p * G)(*key[2]), cap, cap.ctypes.data_as(u64p), tot,
                                     tot.ctypes.data_as(u64p), allv, allv.ctypes.data_as(u64p))
        _, wr, ws, wb, _, cap_p, tot, tot_p, allv, allv_p = xc
        res = _Result()
        rc = _lib.hj_xd_join(self._h, rank, gpu_bits, _ptr(cols[0]), _ptr(cols[1]), cols[0].numel(), _ptr(cols[2]),
                             _ptr(cols[3]), cols[2].numel(), local_bits, out_mode, wr, ws, wb, cap_p, timeout_ms,
                             ctypes.byref(res), tot_p, allv_p)
        tot = tot.copy()
        if rc not in (0, XD_REGROW):
            self._check(rc)
        out = _result(res)
        if rc == 0 and out_mode == OUT_MATERIALIZE and res.matches:
            out.r_pay = _wrap_device(res.r_pay_out, res.matches, self.pay_bytes, dev_)
            out.s_pay = _wrap_device(res.s_pay_out, res.matches, self.pay_bytes, dev_)
        return rc, out, tot, (int(allv[0]), int(allv[1]))


    def xd_reserve(self, gpu_bits: int, nR: int, nS: int, local_bits: int, out_mode: int, win_R_bytes: int,
                   win_S_bytes: int):
        self._check(_lib.hj_xd_reserve(self._h, gpu_bits, nR, nS, local_bits, out_mode, int(win_R_bytes),
                                       int(win_S_bytes)))


def xd_header_bytes(G: int, local_bits: int) -> int:
    return int(_lib.hj_xd_header_bytes(G, local_bits))


def exchange_row_len(G: int, local_bits: int) -> int:
    """Entries per count row of the exchange: 2^b1, the pass-1 digits of one destination."""
    return int(_lib.hj_exchange_row_len(G, local_bits))


def _result(res: _Result) -> JoinResult:
    return JoinResult(matches=int(res.matches), checksum=int(res.checksum), n_items=int(res.n_items),
                      radix_bits=res.radix_bits, passes=res.passes, ms_total=res.ms_total,
                      ms_partition=res.ms_partition, ms_join=res.ms_join,
                      ms_kernel=tuple(res.ms_kernel), kernels=int(res.kernels))


def _as_device_col(t, width: int):
    import torch

    if not isinstance(t, torch.Tensor) or not t.is_cuda:
        raise TypeError("columns must be CUDA tensors (use join_host for host arrays)")
    if t.dim() != 1 or not t.is_contiguous():
        raise ValueError("columns must be 1-D contiguous tensors")
    if t.element_size() != width:
        raise ValueError(f"column has {t.element_size()}-byte elements, expected {width}")
    return t


def _ptr(t):
    return ctypes.c_void_p(t.data_ptr()) if t.numel() else None


def _nptr(a):
    return a.ctypes.data_as(ctypes.c_void_p) if a.size else None


def _wrap_device(addr: int, n: int, width: int, device):
    """Non-owning torch view of ctx-owned device memory (valid until the next call on the ctx)."""
    import torch

    dtype = torch.int32 if width == 4 else torch.int64

    class _CAI:
        __cuda_array_interface__ = {"shape": (int(n),), "typestr": "<i4" if width == 4 else "<i8",
                                    "data": (int(addr), False), "version": 3, "strides": None}

    return torch.as_tensor(_CAI(), device=device).view(dtype)


_tls = threading.local()


def context(device: int = 0, key_bytes: int = 4, pay_bytes: int = 4) -> Context:
    cache = getattr(_tls, "ctx", None)
    if cache is None:
        cache = _tls.ctx = {}
    key = (device, key_bytes, pay_bytes)
    if key not in cache:
        cache[key] = Context(device, key_bytes, pay_bytes)
    return cache[key]


def join(Rk, Rp, Sk, Sp, radix_bits: int = -1, out_mode: int = OUT_COUNT_CHECKSUM) -> JoinResult:
    """R ⋈ S on CUDA tensors with the thread's cached context for (device, widths)."""
    return context(Rk.device.index or 0, Rk.element_size(), Rp.element_size()).join(Rk, Rp, Sk, Sp, radix_bits, out_mode)


def join_host(Rk, Rp, Sk, Sp, radix_bits: int = -1, out_mode: int = OUT_COUNT_CHECKSUM, device: int = 0) -> JoinResult:
    return context(device, Rk.dtype.itemsize, Rp.dtype.itemsize).join_host(Rk, Rp, Sk, Sp, radix_bits, out_mode)


def partition(keys, pays, radix_bits: int):
    return context(keys.device.index or 0, keys.element_size(), pays.element_size()).partition(keys, pays, radix_bits)
