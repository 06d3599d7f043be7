#!/usr/bin/env python
"""Benchmark of the B200 radix-partitioned hash join (DESIGN.md §6 states the contract).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--config c3] [--impl hj|reference]

One step = one hj_join call (all hot-path rows a1-a8) over the workload resident in HBM.
Rank 0 prints ONE JSON line. Metric: (|R|+|S|) tuples/s (§V-A).
Default workload: BASELINE.json config c3 (|R| = |S| = 2^27, 1:1 unique dense keys, 4 B keys
and payloads, materialized output) -- the north star's roofline target.

--impl reference times the CPU oracle (oracle/, the only other place bench.py executes it) on
the box's host cores, on a bounded key-slice of the same workload (each step one slice).
"""
from __future__ import annotations

import argparse
import json
import os
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import workloads as W  # noqa: E402

METRIC = "join throughput (|R|+|S|) tuples/s"
UNIT = "tuples/s"
FALLBACK_HBM_GBS = 6650.0
NOMINAL_HBM_GBS = 8000.0  # the north star's nominal HBM3e figure (reported beside the measured one)


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=50)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--config", default="c3", choices=sorted(W.CONFIGS))
    ap.add_argument("--impl", default="hj", choices=["hj", "reference"])
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--cpu-slice-bits", type=int, default=2, help="cpu_baseline sample = 1 of 2^bits key slices")
    ap.add_argument("--e2e-steps", type=int, default=3)
    ap.add_argument("--clock-period", type=float, default=0.01,
                    help="NVML clock / throttle sampling period (s) during the timed region; 0 = off (testing only)")
    ap.add_argument("--partitioner", default="histogram", choices=["histogram", "bucket-chains"],
                    help="HJ_OPT_PARTITIONER: histogram + exact placement (default) or the paper's bucket chains "
                         "(NEXT-1; more device memory)")
    ap.add_argument("--sync-calls", action="store_true",
                    help="one synchronous hj_join per timed step instead of K queued hj_join_async calls")
    ap.add_argument("--dist", action="store_true", help="use the multi-GPU exchange path even at N=1")
    ap.add_argument("--debug-one-device", action="store_true",
                    help="testing only: every rank on cuda:0 with a gloo process group (validates the multi-rank "
                         "flow on a one-GPU box; not a scaling measurement)")
    ap.add_argument("--exchange", default="direct", choices=["direct", "nccl"],
                    help="multi-GPU exchange: direct = pass 1 stores into the owners' windows over peer memory "
                         "(hj_xd_*); nccl = pack + NCCL all_to_all (hj_exchange_pack)")
    return ap.parse_args()


def peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    return FALLBACK_HBM_GBS, "fallback (B200_PROFILING.md)"


def workload_desc(w: W.Workload) -> str:
    rel = {"fk": "FK uniform", "1to1": "1:1 (S a permutation of R's keys)", "zipf": f"FK Zipf z={w.z}"}[w.dist]
    return (f"{w.name}: |R|={w.nR} |S|={w.nS} {rel}, {w.key_bytes} B keys ({w.keys}) + {w.key_bytes} B payloads, "
            f"{'materialized' if w.out_mode else 'count+checksum'} output, seed {w.seed}")


def alg_bytes(w: W.Workload, matches: int):
    """Algorithmic HBM bytes per step: two partition passes read
    and write every tuple (4w), the join reads every tuple once (w), materialization writes
    2V per match; the histogram reads K per tuple (implementation bytes)."""
    wb = 2 * w.key_bytes
    n = w.n
    out = 2 * w.key_bytes * matches if w.out_mode == 1 else 0
    per_kernel = {"hist": w.key_bytes * n, "plan": 0, "pass1": 2 * wb * n, "pass2": 2 * wb * n, "join": wb * n + out}
    path = 5 * wb * n + out
    return per_kernel, path


class ClockSampler:
    """nvidia-smi-equivalent clock / throttle sampling (NVML) during the timed region."""

    def __init__(self, index: int, period_s: float = 0.01):
        self.samples, self.reasons, self.max_mhz = [], set(), None
        self.period = period_s
        self._stop = threading.Event()
        try:
            import pynvml

            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(index)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
        except Exception as e:  # pragma: no cover
            self.nv = None
            self.err = str(e)

    def _run(self):
        nv = self.nv
        names = {
            "hw_slowdown": getattr(nv, "nvmlClocksThrottleReasonHwSlowdown", 0x8),
            "sw_thermal_slowdown": getattr(nv, "nvmlClocksThrottleReasonSwThermalSlowdown", 0x20),
            "hw_thermal_slowdown": getattr(nv, "nvmlClocksThrottleReasonHwThermalSlowdown", 0x40),
            "sw_power_cap": getattr(nv, "nvmlClocksThrottleReasonSwPowerCap", 0x4),
            "hw_power_brake_slowdown": getattr(nv, "nvmlClocksThrottleReasonHwPowerBrakeSlowdown", 0x80),
        }
        while not self._stop.is_set():
            try:
                self.samples.append(nv.nvmlDeviceGetClockInfo(self.h, nv.NVML_CLOCK_SM))
                r = nv.nvmlDeviceGetCurrentClocksThrottleReasons(self.h)
                for k, bit in names.items():
                    if r & bit:
                        self.reasons.add(k)
            except Exception:
                pass
            time.sleep(self.period)

    def __enter__(self):
        if self.nv and self.period <= 0:  # testing only: no sampling
            self.nv = None
            self.err = "sampling disabled (--clock-period 0)"
        if self.nv:
            self.t = threading.Thread(target=self._run, daemon=True)
            self.t.start()
        return self

    def __exit__(self, *a):
        if self.nv:
            self._stop.set()
            self.t.join()

    def summary(self):
        if not self.nv:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": [], "error": getattr(self, "err", "")}
        med = float(np.median(self.samples)) if self.samples else None
        return {"sm_mhz": med, "sm_max_mhz": self.max_mhz, "reasons": sorted(self.reasons), "samples": len(self.samples)}


def dist_env(one_device: bool = False):
    ws = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = 0 if one_device else int(os.environ.get("LOCAL_RANK", "0"))
    return ws, rank, local


def key_slices(w: W.Workload, Rk, Rp, Sk, Sp, slices: int):
    """Split both relations by the top log2(slices) bits of fmix64(key) (untimed setup). The join
    decomposes exactly over any key partition, so every slice is a bounded,
    representative sample of the same workload."""
    bits = slices.bit_length() - 1
    hR = (W.np_fmix64(Rk.astype(np.uint64)) >> np.uint64(64 - bits)).astype(np.int64)
    hS = (W.np_fmix64(Sk.astype(np.uint64)) >> np.uint64(64 - bits)).astype(np.int64)
    oR, oS = np.argsort(hR, kind="stable"), np.argsort(hS, kind="stable")
    cR, cS = np.bincount(hR, minlength=slices), np.bincount(hS, minlength=slices)
    bR, bS = np.concatenate([[0], np.cumsum(cR)]), np.concatenate([[0], np.cumsum(cS)])
    Rk, Rp, Sk, Sp = Rk[oR], Rp[oR], Sk[oS], Sp[oS]
    return [(Rk[bR[t]:bR[t + 1]], Rp[bR[t]:bR[t + 1]], Sk[bS[t]:bS[t + 1]], Sp[bS[t]:bS[t + 1]])
            for t in range(slices)]


def cpu_model() -> str:
    try:
        for line in open("/proc/cpuinfo"):
            if line.startswith("model name"):
                return line.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


class PinnedCore:
    """Run the (single-threaded) oracle pinned to one host core, like `taskset -c <core>`."""

    def __init__(self, core: int = 0):
        self.core = core

    def __enter__(self):
        try:
            self.prev = os.sched_getaffinity(0)
            cores = sorted(self.prev)
            self.core = self.core if self.core in self.prev else cores[0]
            os.sched_setaffinity(0, {self.core})
            self.pinned = True
        except (AttributeError, OSError):
            self.pinned = False
        return self

    def __exit__(self, *a):
        if self.pinned:
            os.sched_setaffinity(0, self.prev)


def cpu_oracle_sample(w: W.Workload, Rk, Rp, Sk, Sp, slices: int):
    """Time the oracle (as it stands, single thread, pinned to one core) on key slice 0 of
    `slices` of the workload (pre-filtered, untimed); throughput = (|R|+|S|) / (slices * t_slice)."""
    import oracle

    sl = key_slices(w, Rk, Rp, Sk, Sp, slices)[0]
    with PinnedCore(0) as pin:
        t0 = time.perf_counter()
        res = oracle.hash_join(*sl, materialize=bool(w.out_mode))
        dt = time.perf_counter() - t0
    v = w.n / (slices * dt)
    sample = (f"key slice 0 of {slices} (top bits of fmix64(key), pre-filtered) of the full {w.name} input: "
              f"|R|={len(sl[0])} |S|={len(sl[2])}, {'materialized' if w.out_mode else 'count'}, {res[0]} matches in "
              f"{dt:.2f} s; value = (|R|+|S|)/({slices}*t_slice)")
    return {"value": v, "unit": UNIT, "cores": 1, "kind": "oracle", "sample": sample, "host_cpus": os.cpu_count(),
            "cpu_model": cpu_model(), "pinned_core": pin.core if pin.pinned else None}


def closed_form(w: W.Workload):
    """(matches, checksum) the generator fixes for FK / 1:1 / Zipf-FK inputs:
    every S row j matches exactly R row rho(j), so matches = |S| and checksum = sum_j sig(rho(j), j)
    (sig = fmix64(r_pay ^ s_pay * golden), payloads are row ids). Computed on the host, untimed;
    every timed step's result is compared with it."""
    j = np.arange(w.nS, dtype=np.uint64)
    cdf = W.zipf_cdf(w.nR, w.z) if w.dist == "zipf" else None
    rho = W.np_rho_for(w, j, cdf)
    with np.errstate(over="ignore"):
        chk = int(W.np_fmix64(rho ^ (j * np.uint64(0x9E3779B97F4A7C15))).sum(dtype=np.uint64))
    return w.nS, chk


def run_reference(args, w: W.Workload):
    ws, rank, _ = dist_env()
    if rank != 0:
        return
    import oracle

    oracle.build()
    Rk, Rp, Sk, Sp = W.np_generate(w)
    # each step joins one key slice; the slice count keeps the whole run near 2.5 min of oracle
    # time assuming ~60 s for the full join (single core)
    steps = args.warmup + args.steps
    slices = 1
    while slices < max(4, 60.0 * steps / 150.0):
        slices *= 2
    parts = key_slices(w, Rk, Rp, Sk, Sp, slices)
    del Rk, Rp, Sk, Sp
    times = []
    with PinnedCore(0) as pin:
        for i in range(steps):
            t0 = time.perf_counter()
            oracle.hash_join(*parts[i % slices], materialize=bool(w.out_mode))
            if i >= args.warmup:
                times.append(time.perf_counter() - t0)
    t = float(np.mean(times))
    v = w.n / (slices * t)
    cpu = {"value": v, "unit": UNIT, "cores": 1, "kind": "oracle", "host_cpus": os.cpu_count(),
           "cpu_model": cpu_model(), "pinned_core": pin.core if pin.pinned else None,
           "sample": f"each step one key slice (1 of {slices}, top bits of fmix64(key), pre-filtered) of the full "
                     f"{w.name} input; value = (|R|+|S|)/({slices}*mean t_slice)"}
    print(json.dumps({"impl": "reference", "metric": METRIC, "value": v, "unit": UNIT, "n_gpus": ws,
                      "steps": args.steps, "warmup": args.warmup, "ms_per_step": t * 1e3, "higher_is_better": True,
                      "scaling": "weak", "vs_baseline": None, "dtype": "u32" if w.key_bytes == 4 else "u64",
                      "data": "synthetic", "config": {"workload": workload_desc(w)}, "cpu_baseline": cpu,
                      "e2e": {"value": v, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}),
          flush=True)


def main():
    args = parse()
    w = W.CONFIGS[args.config]
    if args.impl == "reference":
        return run_reference(args, w)

    import torch

    ws, rank, local = dist_env(args.debug_one_device)
    use_dist = ws > 1 or args.dist
    if use_dist:
        import torch.distributed as dist

        torch.cuda.set_device(local)
        if ws == 1:
            os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
            os.environ.setdefault("MASTER_PORT", "29531")
            os.environ.setdefault("RANK", "0")
            os.environ.setdefault("WORLD_SIZE", "1")
        dist.init_process_group("gloo" if args.debug_one_device else "nccl")
    dev = torch.device("cuda", local)
    torch.cuda.set_device(dev)
    import paper_conf_icde_sioulasckaa19_b200 as hj

    ctx = hj.Context(local, w.key_bytes, w.key_bytes)
    if args.partitioner == "bucket-chains":
        ctx.set_option(hj.OPT_PARTITIONER, 1)
    Rk, Rp, Sk, Sp = W.torch_generate(w, device=dev)
    if ws > 1:
        # strong scaling: the same workload, rows sharded across ranks (inputs start row-sharded)
        rs = slice(rank * w.nR // ws, (rank + 1) * w.nR // ws)
        ss = slice(rank * w.nS // ws, (rank + 1) * w.nS // ws)
        Rk, Rp, Sk, Sp = (t[sl].contiguous() for t, sl in ((Rk, rs), (Rp, rs), (Sk, ss), (Sp, ss)))
    torch.cuda.synchronize()
    stream = torch.cuda.current_stream(dev)
    from paper_conf_icde_sioulasckaa19_b200 import dist as hjdist

    # the local radix bits of the exchange path, fixed once (the whole workload's |R| is known)
    local_bits = hjdist._local_bits(w.nR, ws)

    def step():
        if not use_dist:
            return ctx.join(Rk, Rp, Sk, Sp, radix_bits=w.radix_bits, out_mode=w.out_mode)
        return hjdist.join(Rk, Rp, Sk, Sp, local_bits=local_bits, out_mode=w.out_mode, ctx=ctx,
                           exchange=args.exchange)

    exchange_note = None
    if use_dist and args.exchange == "direct":
        # the direct store needs every peer's windows mapped through CUDA IPC; where a launcher
        # hides the peers' devices that cannot work: then every rank switches to the NCCL
        # all-to-all exchange together (decided by an all-reduce, so no rank is left waiting)
        ok = torch.ones(1, device="cpu" if args.debug_one_device else dev)
        try:
            step()
        except Exception as e:  # HJError from hj_ipc_open / hj_xd_join
            ok.zero_()
            exchange_note = f"direct store unavailable ({str(e)[:120]}); NCCL all_to_all used"
        torch.distributed.all_reduce(ok, op=torch.distributed.ReduceOp.MIN)
        if ok.item() == 0:
            args.exchange = "nccl"
            exchange_note = exchange_note or "direct store unavailable on a peer; NCCL all_to_all used"
    expect = closed_form(w)  # untimed; every step below is checked against it
    for _ in range(args.warmup):
        res = step()
        assert (res.matches, res.checksum) == expect, ("closed form", res.matches, res.checksum, expect)

    def barrier():
        if use_dist:
            torch.distributed.barrier()
        torch.cuda.synchronize()

    per_k = np.zeros(5)
    launches = 0
    sent = 0
    barrier()
    with ClockSampler(local, args.clock_period) as clk:
        e0 = torch.cuda.Event(enable_timing=True)
        e1 = torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        results = []
        if not use_dist and not args.sync_calls:
            # hj_join_async: the K joins are queued back to back on the stream (each call's host
            # preparation overlaps the previous call's kernels); hj_sync returns every step's result
            for _ in range(args.steps):
                ctx.join_async(Rk, Rp, Sk, Sp, radix_bits=w.radix_bits, out_mode=w.out_mode)
            e1.record(stream)
            outs = ctx.sync()
        else:
            outs = [step() for _ in range(args.steps)]
            e1.record(stream)
        for res in outs:
            results.append((res.matches, res.checksum))
            loc = res if not use_dist else res.local
            per_k += np.array(loc.ms_kernel)
            # + the sender side: direct = hist, plan, count rows, pass 1, barrier; nccl = (hist, plan, pass 1) x 2
            launches += loc.kernels if not use_dist else loc.kernels + (5 if args.exchange == "direct" else 6)
            sent += 0 if not use_dist else res.sent_bytes
        barrier()
    bad = [k for k, r in enumerate(results) if r != expect]
    assert not bad, f"timed steps {bad[:5]} differ from the closed form {expect}"
    ms = e0.elapsed_time(e1) / args.steps
    if use_dist:
        t = torch.tensor([ms], device="cpu" if args.debug_one_device else dev)
        torch.distributed.all_reduce(t, op=torch.distributed.ReduceOp.MAX)
        ms = float(t.item())
    per_k /= args.steps
    value = w.n / (ms * 1e-3)  # the whole workload's tuples (sharded across ranks when ws > 1)

    if rank != 0:
        if use_dist:
            torch.distributed.destroy_process_group()
        return

    peak, peak_src = peaks()
    kb, path_bytes = alg_bytes(w, res.matches)  # res.matches: the whole join's (all ranks)
    names = ["hist", "plan", "pass1", "pass2", "join"]
    kms = dict(zip(names, per_k.tolist()))
    dom = max(names, key=lambda k: kms[k])
    traffic = None
    tf = os.path.join(ROOT, "profiles", f"traffic_{w.name}.json")
    if os.path.exists(tf):
        traffic = json.load(open(tf)).get(dom)
    ach = kb[dom] / (kms[dom] * 1e-3) / 1e9
    roof = {"bound": "hbm", "kernel": dom, "achieved": ach, "peak": peak, "unit": "GB/s", "frac": ach / peak,
            "traffic": traffic, "alg_bytes_per_launch": kb[dom], "ms_per_launch": kms[dom], "peak_source": peak_src}
    path_ach = path_bytes / (ms * 1e-3) / 1e9
    roof_path = {"bound": "hbm", "achieved": path_ach, "peak": peak, "unit": "GB/s", "frac": path_ach / peak,
                 "frac_nominal_8tbs": path_ach / NOMINAL_HBM_GBS,
                 "alg_bytes_per_step": path_bytes,
                 "kernel_fracs": {k: (kb[k] / (kms[k] * 1e-3) / 1e9 / peak if kms[k] > 0.01 and kb[k] else None)
                                  for k in names}}

    out = {"metric": METRIC, "value": value, "unit": UNIT, "n_gpus": ws, "steps": args.steps, "warmup": args.warmup,
           "ms_per_step": ms, "higher_is_better": True, "scaling": "weak" if ws == 1 else "strong",
           "vs_baseline": None,
           "dtype": "u32" if w.key_bytes == 4 else "u64", "data": "synthetic",
           "config": {"workload": workload_desc(w), "radix_bits": loc.radix_bits, "passes": loc.passes,
                      "join_items": loc.n_items,
                      "l2": "inputs larger than L2 (2 GiB in + 4 GiB partition buffers vs 126 MB L2); no flush",
                      "partitioner": args.partitioner,
                      "calls": ("hj_join_async x K queued on the stream, one hj_sync; every step's result "
                                "returned and validated" if not use_dist and not args.sync_calls else
                                "one synchronous call per step"),
                      "parallelism": "1 GPU" if not use_dist else
                      f"{ws} rank(s): rows sharded, radix exchange "
                      + ("fused into pass 1 (direct peer stores, hj_xd_*)" if args.exchange == "direct"
                         else "over NCCL all_to_all") + ", per-rank 2-pass join"},
           "roofline": roof, "roofline_path": roof_path, "kernels_ms": kms, "clocks": clk.summary(),
           "gpu_launches": launches,
           "validated": f"every warm-up and timed step: (matches, checksum) == closed form {list(expect)}"}
    if use_dist:
        out["config"]["exchange"] = args.exchange + (f" ({exchange_note})" if exchange_note else "")
    if use_dist:
        out["nvlink"] = {"bytes_sent_per_gpu_per_step": sent / args.steps,
                         "achieved_GBps": sent / args.steps / (ms * 1e-3) / 1e9, "peak_GBps": 900.0,
                         "note": "tuple bytes rank 0 sent to other ranks / step time; "
                                 + ("pass-1 peer stores over NVLink (CUDA IPC mappings)" if args.exchange == "direct"
                                    else "all_to_all_single over NCCL")}

    if not args.no_e2e and not use_dist:
        # end to end through the public API from pinned host memory: H2D of the inputs, the join,
        # D2H of the result (matches/checksum, and the materialized pairs) every step
        hcols = []
        for t in (Rk, Rp, Sk, Sp):
            h = torch.empty(t.shape, dtype=t.dtype, pin_memory=True)
            h.copy_(t)
            hcols.append(h.numpy())
        ctx.join_host(*hcols, radix_bits=w.radix_bits, out_mode=w.out_mode, copy=False)
        t0 = time.perf_counter()
        for _ in range(args.e2e_steps):
            r2 = ctx.join_host(*hcols, radix_bits=w.radix_bits, out_mode=w.out_mode, copy=False)
        dt = (time.perf_counter() - t0) / args.e2e_steps
        assert (r2.matches, r2.checksum) == (res.matches, res.checksum)
        out["e2e"] = {"value": w.n / dt, "unit": UNIT, "h2d_bytes_per_step": int(sum(h.nbytes for h in hcols)),
                      "d2h_bytes_per_step": 16 + (2 * w.key_bytes * r2.matches if w.out_mode else 0),
                      "ms_per_step": dt * 1e3, "steps": args.e2e_steps, "api": "hj_join_host (pinned host columns)"}
        del hcols

    if not args.no_cpu_baseline and ws == 1 and not use_dist:
        host = [t.cpu().numpy().view(np.uint32 if w.key_bytes == 4 else np.uint64) for t in (Rk, Rp, Sk, Sp)]
        out["cpu_baseline"] = cpu_oracle_sample(w, *host, slices=1 << args.cpu_slice_bits)
    print(json.dumps(out), flush=True)
    if use_dist:
        torch.distributed.destroy_process_group()


if __name__ == "__main__":
    main()
