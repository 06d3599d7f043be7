"""Histogram path vs the paper's bucket chains (NEXT-1, HJ_OPT_PARTITIONER = 1) on the bench configs.

    python tools/bc_compare.py [config ...]     (default: c3 c2 c4_z1.5 c5_gpu)

Per config and partitioner (bucket chains with the warp-specialized passes, and with the
lock-step k_pass): mean ms_total (device events of hj_join) over 10 calls after 3 warm-up
calls, the per-kernel split, and the result (matches, checksum) -- the two partitioners must agree.
"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402
import paper_conf_icde_sioulasckaa19_b200 as hj  # noqa: E402
import workloads as W  # noqa: E402


def main():
    names = sys.argv[1:] or ["c3", "c2", "c4_z1.5", "c5_gpu"]
    print("| config | partitioner | ms_total | kernels ms | matches |")
    print("|---|---|---|---|---|")
    for name in names:
        w = W.CONFIGS[name]
        cols = W.torch_generate(w, device="cuda")
        res = {}
        for part, ws in ((0, 1), (1, 1), (1, 0)):
            ctx = hj.Context(0, w.key_bytes, w.key_bytes)
            ctx.set_option(hj.OPT_PARTITIONER, part)
            ctx.set_option(hj.OPT_PASS_WS, ws)
            for _ in range(3):
                r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
            ms, km = 0.0, None
            for _ in range(10):
                r = ctx.join(*cols, radix_bits=w.radix_bits, out_mode=w.out_mode)
                ms += r.ms_total
                k = list(r.ms_kernel)
                km = k if km is None else [a + b for a, b in zip(km, k)]
            torch.cuda.synchronize()
            res[(part, ws)] = (r.matches, r.checksum)
            arm = ("bucket chains" if part else "histogram") + (" (lock-step passes)" if not ws else "")
            print(f"| {name} | {arm} | {ms / 10:.3f} | "
                  f"{' '.join(f'{x / 10:.3f}' for x in km)} | {r.matches} |", flush=True)
            ctx.close()
        assert len(set(res.values())) == 1, (name, res)
        del cols
        torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
