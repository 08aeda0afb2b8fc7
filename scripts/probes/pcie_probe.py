"""H2D / D2H copy rates from pinned memory: one stream vs several (diagnostic
for bench.py's e2e leg)."""
import torch

N = 1 << 24  # 64 MiB fp32 per array
h = [torch.empty(N, dtype=torch.float32).pin_memory() for _ in range(4)]
d = [torch.empty(N, dtype=torch.float32, device="cuda") for _ in range(4)]
hx = torch.empty(N, dtype=torch.float32).pin_memory()
dx = torch.empty(N, dtype=torch.float32, device="cuda")
streams = [torch.cuda.Stream() for _ in range(5)]


def run(nstreams, with_d2h, reps=10):
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    e0.record()
    for _ in range(reps):
        for q in range(4):
            s = streams[q % nstreams]
            s.wait_event(e0)
            with torch.cuda.stream(s):
                d[q].copy_(h[q], non_blocking=True)
        if with_d2h:
            s = streams[4]
            s.wait_event(e0)
            with torch.cuda.stream(s):
                hx.copy_(dx, non_blocking=True)
    for s in streams:
        torch.cuda.current_stream().wait_stream(s)
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1) / reps
    return 4 * N * 4 / ms / 1e6, ms


for ns in (1, 2, 4):
    for dd in (False, True):
        gbs, ms = run(ns, dd)
        print(f"H2D 4 x 64 MiB on {ns} stream(s){' + concurrent 64 MiB D2H' if dd else ''}: {ms:.2f} ms/step, "
              f"H2D {gbs:.1f} GB/s", flush=True)
