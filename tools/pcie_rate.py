import torch, time
n = 1 << 30
h = torch.empty(n, dtype=torch.uint8, pin_memory=True); d = torch.empty(n, dtype=torch.uint8, device="cuda")
h2 = torch.empty(n, dtype=torch.uint8, pin_memory=True)
for _ in range(2): d.copy_(h, non_blocking=True); torch.cuda.synchronize()
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
e0.record(); [d.copy_(h, non_blocking=True) for _ in range(4)]; e1.record(); torch.cuda.synchronize()
print("H2D GB/s", 4 * n / e0.elapsed_time(e1) / 1e6)
e0.record(); [h2.copy_(d, non_blocking=True) for _ in range(4)]; e1.record(); torch.cuda.synchronize()
print("D2H GB/s", 4 * n / e0.elapsed_time(e1) / 1e6)
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
torch.cuda.synchronize(); t0 = time.perf_counter()
with torch.cuda.stream(s1): [d.copy_(h, non_blocking=True) for _ in range(4)]
with torch.cuda.stream(s2):
    d2 = torch.empty(n, dtype=torch.uint8, device="cuda"); [h2.copy_(d2, non_blocking=True) for _ in range(2)]
torch.cuda.synchronize(); dt = time.perf_counter() - t0
print("bidirectional: 4 GiB H2D + 2 GiB D2H in", dt * 1e3, "ms")
