import torch
x = torch.ones(8 * (1 << 20), device="cuda")      # 32 MB
y = torch.empty_like(x)
z = torch.ones(16 * (1 << 20), device="cuda")     # 64 MB
w = torch.empty_like(z)
torch.cuda.synchronize()
for _ in range(2):
    torch.mul(x, 2.0, out=y)   # reads x (32 MB)
    torch.mul(x, 3.0, out=y)   # re-reads x: L2?
    torch.mul(z, 2.0, out=w)   # 64 MB
    torch.mul(z, 3.0, out=w)
torch.cuda.synchronize()
