import sys, os; sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import os, numpy as np, torch, lmgen, oracle
import paper_conf_ipps_steuwerkg12_b200 as pkg
name=os.environ.get('DBG_CFG','C1'); slabs=int(os.environ.get('DBG_SLABS','2'))
cfg=lmgen.CONFIGS[name]
n=cfg.n_events if name=='C1' else 50000
ev=lmgen.subset_events(cfg,1,n)
g=oracle.geom(cfg.dims,cfg.voxel_mm)
f0=np.random.default_rng(3).uniform(0.5,2.0,cfg.n_voxels).astype(np.float32)
ref=oracle.error_image(g,ev,f0)
rec=pkg.Reconstructor(cfg.dims,cfg.voxel_mm,torch.ones(cfg.n_voxels,device='cuda'))
rec.set_slabs(slabs)
c=torch.zeros(cfg.n_voxels,device='cuda')
rec.error_image(torch.from_numpy(ev).cuda(),torch.from_numpy(f0).cuda(),c); rec.synchronize()
got=c.cpu().numpy().astype(np.float64)
err=np.abs(got-ref); print(name, slabs, 'zlist',os.environ.get('LMOSEM_ZLIST'),'zmed',os.environ.get('LMOSEM_ZMED'),'max abs err',err.max(),'ref max',ref.max(), 'sum got/ref', got.sum()/ref.sum())
