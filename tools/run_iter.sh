SWEEP="C B" bash tools/gpu_quick.sh
bash tools/gpu_prof.sh xplanC C xplan
