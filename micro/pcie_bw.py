"""Pinned host <-> device copy bandwidth for 2 GiB (the c2 records), each direction alone and
both at once on two streams: the bound of bench.py's e2e number."""
import torch

nb = 2 << 30
h_in = torch.empty(nb, dtype=torch.uint8, pin_memory=True)
h_out = torch.empty(nb, dtype=torch.uint8, pin_memory=True)
d_a = torch.empty(nb, dtype=torch.uint8, device="cuda")
d_b = torch.empty(nb, dtype=torch.uint8, device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()


def timed(fn, reps=5):
    fn()
    torch.cuda.synchronize()
    st, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    st.record()
    for _ in range(reps):
        fn()
    en.record()
    torch.cuda.synchronize()
    return st.elapsed_time(en) / reps


def both():
    ev = torch.cuda.Event()
    ev.record()
    s1.wait_event(ev)
    s2.wait_event(ev)
    with torch.cuda.stream(s1):
        d_a.copy_(h_in, non_blocking=True)
    with torch.cuda.stream(s2):
        h_out.copy_(d_b, non_blocking=True)
    torch.cuda.current_stream().wait_stream(s1)
    torch.cuda.current_stream().wait_stream(s2)


t_h2d = timed(lambda: d_a.copy_(h_in, non_blocking=True))
t_d2h = timed(lambda: h_out.copy_(d_b, non_blocking=True))
t_both = timed(both)
print(f"H2D 2 GiB: {t_h2d:.2f} ms ({nb / t_h2d / 1e6:.1f} GB/s)")
print(f"D2H 2 GiB: {t_d2h:.2f} ms ({nb / t_d2h / 1e6:.1f} GB/s)")
print(f"H2D + D2H concurrently, 2 GiB each: {t_both:.2f} ms ({2 * nb / t_both / 1e6:.1f} GB/s total)")
