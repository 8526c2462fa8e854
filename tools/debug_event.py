"""Diagnostic: per-voxel chord lengths of the worst forward-projection event, GPU vs oracle."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
import oracle, paper_conf_ipps_steuwerkg12_b200 as pkg
dims, vox = (33, 5, 64), (0.6, 2.0, 0.45)
g = oracle.geom(dims, vox)
V = int(np.prod(dims)); half = 0.5 * np.asarray(dims) * np.asarray(vox)
rng = np.random.default_rng(sum(dims)); n = 3000
c = rng.uniform(-half, half, (n, 3)); d = rng.normal(size=(n, 3)); d /= np.linalg.norm(d, axis=1, keepdims=True)
r = rng.uniform(0.2, 1.5, (n, 1)) * np.linalg.norm(half)
ev = np.concatenate([c - r * d, c + r * d], axis=1).astype(np.float32)
s = rng.uniform(0.5, 1.0, V).astype(np.float32); f0 = rng.uniform(0.5, 2.0, V).astype(np.float32)
rec = pkg.Reconstructor(dims, vox, torch.from_numpy(s).cuda())
fp = torch.empty(n, device="cuda"); rec.forward(torch.from_numpy(ev).cuda(), torch.from_numpy(f0).cuda(), fp)
ref = oracle.forward(g, ev, f0); got = fp.cpu().numpy()
rel = np.abs(got - ref) / ref; i = int(np.argmax(rel)); print("worst event", i, ev[i], "rel", rel[i], "fp", ref[i], got[i])
ones = torch.ones(V, device="cuda"); cc = torch.empty(V, device="cuda")
e1 = torch.from_numpy(ev[i:i + 1].copy()).cuda(); rec.error_image(e1, ones, cc)
fp1 = torch.empty(1, device="cuda"); rec.forward(e1, ones, fp1)
a_gpu = cc.cpu().numpy().astype(np.float64) * fp1.item()
co, ln = oracle.siddon_path(g, ev[i, :3].astype(float), ev[i, 3:].astype(float))
print("oracle pieces", len(co), "chord", ln.sum(), "gpu chord", fp1.item())
exp = np.zeros(V); exp[co] = ln
diff = np.abs(a_gpu - exp); k = np.argsort(-diff)[:12]
for j in k: print(j, np.unravel_index(j, dims[::-1])[::-1], exp[j], a_gpu[j], diff[j])
