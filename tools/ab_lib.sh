cd /root/repo
for i in 1 2; do
for L in paper_conf_cluster_luzw20_b200/libconv2d_old.so paper_conf_cluster_luzw20_b200/libconv2d.so; do
echo $L; C2D_LIB=$L timeout 300 python tools/variants.py --sizes 8192,4096 --ks 7,11,15 --variants 0 2>&1 | tail -6
done; done
