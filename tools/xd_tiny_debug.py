import os, sys, numpy as np, torch, concurrent.futures as cf
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
sys.path.insert(0, os.getcwd()); sys.path.insert(0, os.path.join(os.getcwd(), "tests"))
import paper_conf_icde_sioulasckaa19_b200 as hj, workloads as W, oracle
from test_dist import _xd_join_threads
import test_dist
w = W.Workload("tiny", 3, 5000, "fk", keys="sparse", seed=199)
G, lb = 4, 2
cols = W.np_generate(w)
shards = []
for v in range(G):
    rs = slice(v * w.nR // G, (v + 1) * w.nR // G); ss = slice(v * w.nS // G, (v + 1) * w.nS // G)
    shards.append([torch.from_numpy(a[sl].view(np.int32).copy()).cuda() for a, sl in zip(cols, (rs, rs, ss, ss))])
ctxs = [hj.Context(0, 4, 4) for _ in range(G)]
streams = [torch.cuda.Stream() for _ in range(G)]
H = hj.xd_header_bytes(G, lb)
cap = np.zeros((2, G), dtype=np.uint64); win = [[0] * G for _ in range(3)]
for v in range(G):
    for r, n in ((0, w.nR), (1, w.nS)):
        cap[r, v] = H + 64 + int(8 * n / G + 16) * 8
        win[r][v], _, _ = ctxs[v].xd_window(r, int(cap[r, v]), want_handle=False)
    win[2][v], _, _ = ctxs[v].xd_window(2, hj.XD_BOARD_BYTES, want_handle=False)
for v in range(G):
    ctxs[v].xd_reserve(2, shards[v][0].numel(), shards[v][2].numel(), lb, 0, cap[0, v], cap[1, v])
torch.cuda.synchronize()
def call(v):
    try:
        with torch.cuda.stream(streams[v]):
            return ctxs[v].xd_join(v, 2, *shards[v], lb, 0, win[0], win[1], win[2], cap, 5000)[::3]
    except Exception as e:
        return repr(e)
with cf.ThreadPoolExecutor(G) as ex:
    print(list(ex.map(call, range(G))), oracle.hash_join(*cols))
torch.cuda.synchronize()
for v in range(G):
    b = hj._wrap_device(win[2][v], 192, 8, torch.device("cuda", 0)).cpu().numpy()
    print("board", v, "B", b[0:G], "A", b[64:64 + G], "C", b[128:128 + G])
